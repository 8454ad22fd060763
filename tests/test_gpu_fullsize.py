"""Full BASELINE.json sizes (2^28 records) in the launch configuration bench.py times.

The oracle cannot sort 2^28 records in seconds, so these check properties that
characterise the unique stable sort at any size ("O(n) certificate"):
with values = input index, the output is THE stable sort iff
  (i)  every value is < n,
  (ii) keys_out[i] == keys_in[vals_out[i]],
  (iii) (sk(keys_out[i]), vals_out[i]) is strictly increasing in i.
Plus sampled oracle checks: the first-digit histogram of the input (oracle) must
equal the run lengths of the first digit in the output."""
import numpy as np
import pytest
import torch

import gen
import oracle

pytestmark = pytest.mark.gpu
DEV = "cuda:0"


def _as_i64(t: torch.Tensor) -> torch.Tensor:
    """Unsigned keys -> int64 preserving unsigned order (sign-bit flip for u64)."""
    if t.dtype == torch.uint32:
        return t.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    x = t.view(torch.int64)
    return x ^ torch.tensor(-(1 << 63), dtype=torch.int64, device=t.device)


def certificate(keys_in, keys_out, vals_out, begin, end):
    n = keys_in.numel()
    kb = 8 * keys_in.element_size()
    idx = _as_i64(vals_out) if vals_out.dtype == torch.uint32 else vals_out.view(torch.int64)
    assert int(idx.min()) >= 0 and int(idx.max()) < n, "values are not input indices"
    g = keys_in.view(torch.int32 if kb == 32 else torch.int64)[idx]
    assert torch.equal(g, keys_out.view(torch.int32 if kb == 32 else torch.int64)), "keys_out != keys_in[vals_out]"
    if kb == 32:
        sk = _as_i64(keys_out)
        sk = (sk >> begin) & ((1 << (end - begin)) - 1)
    else:
        raw = keys_out.view(torch.int64)
        w = end - begin
        sh = (raw >> begin) & ((1 << (64 - begin)) - 1) if begin else raw
        if w < 64:
            sk = sh & ((1 << w) - 1) if w < 63 else sh & 0x7FFFFFFFFFFFFFFF
        else:
            sk = _as_i64(keys_out)
    a, b = sk[:-1], sk[1:]
    ok = (a < b) | ((a == b) & (idx[:-1] < idx[1:]))
    assert bool(ok.all()), f"order/stability violated at {int((~ok).nonzero()[0])}"


def _sort(kd, vd):
    import paper_1611_01137_b200 as hrs
    kb = kd.element_size()
    vb = vd.element_size()
    temp = torch.empty(hrs.temp_bytes(kd.numel(), kb, vb), dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort(kd, vd, temp=temp)
    torch.cuda.synchronize()
    return ko, vo, hrs.get_stats(temp)


def _top_digit_runs(keys_out, kbits):
    top = (_as_i64(keys_out) >> (kbits - 8)) & 0xFF if kbits == 32 else \
        ((keys_out.view(torch.int64) >> 56) & 0xFF)
    return torch.bincount(top, minlength=256).cpu().numpy().astype(np.uint64), top


@pytest.mark.parametrize("dist", ["uniform", "and2", "and3", "and4", "const"])
def test_c2_c3_pairs_u32(dist):
    n = 1 << 28
    k = gen.keys(n, 32, dist, device=DEV)
    v = gen.values(n, 32, "index", device=DEV)
    ko, vo, st = _sort(k, v)
    certificate(k, ko, vo, 0, 32)
    assert st["overflow"] == 0
    # sampled oracle parity: first-digit histogram of the input (oracle) == output runs
    hist, top = _top_digit_runs(ko, 32)
    assert np.array_equal(hist, oracle.histogram(k.cpu(), 24, 32))
    assert bool((top[1:] >= top[:-1]).all())
    if dist == "uniform":
        # predicted structure: two counting passes, then 65536 local sorts
        assert st["counting_passes"] == 2 and st["recs_in_pass"] == [n, n]
        assert st["local_recs"] == n and st["bytes_min"] == 56 * n


@pytest.mark.parametrize("dist", ["uniform", "and2", "and3", "and4", "const"])
def test_c4_pairs_u64(dist):
    n = 1 << 28
    k = gen.keys(n, 64, dist, device=DEV)
    v = gen.values(n, 64, "index", device=DEV)
    ko, vo, st = _sort(k, v)
    certificate(k, ko, vo, 0, 64)
    assert st["overflow"] == 0
    hist, _ = _top_digit_runs(ko, 64)
    assert np.array_equal(hist, oracle.histogram(k.cpu(), 56, 64))
    if dist == "uniform":
        assert st["counting_passes"] == 2 and st["bytes_min"] == 112 * n


def test_c1_keys_only_full_oracle():
    import paper_1611_01137_b200 as hrs
    n = 1 << 20
    k = gen.keys(n, 32, "uniform")
    ko, _ = hrs.sort(k.to(DEV))
    ek, _ = oracle.sort(k, None, 0, 32)
    assert np.array_equal(oracle._u64(ko.cpu()), ek)


def test_large_random_values_slice_parity():
    """2^24 u32/u32 pairs with random values: element-by-element against the oracle."""
    import paper_1611_01137_b200 as hrs
    n = 1 << 24
    k = gen.keys(n, 32, "and2", seed=gen.SEEDS[1])
    v = gen.values(n, 32, "random", seed=gen.SEEDS[1])
    ko, vo = hrs.sort(k.to(DEV), v.to(DEV))
    ek, ev = oracle.sort(k, v, 0, 32)
    assert np.array_equal(oracle._u64(ko.cpu()), ek)
    assert np.array_equal(oracle._u64(vo.cpu()), ev)


def test_more_than_2_31_records():
    """n = 2^31 + 12345 u32/u32 (48 GB with outputs and temp): 64-bit bucket and tile
    offsets, record indices past 2^31.  O(n) certificate, chunked to bound memory."""
    import paper_1611_01137_b200 as hrs
    n = (1 << 31) + 12345
    kd = gen.keys(n, 32, "uniform", device=DEV)
    vd = gen.values(n, 32, "index", device=DEV)
    temp = torch.empty(hrs.temp_bytes(n, 4, 4), dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort(kd, vd, temp=temp)
    torch.cuda.synchronize()
    st = hrs.get_stats(temp)
    del temp
    assert st["counting_passes"] == 3 and st["overflow"] == 0
    ki = kd.view(torch.int32)
    C = 1 << 27
    for a in range(0, n, C):
        b = min(n, a + C + 1)  # one element of overlap with the next chunk
        idx = vo[a:b].view(torch.int32).to(torch.int64) & 0xFFFFFFFF
        assert int(idx.max()) < n
        assert torch.equal(ki[idx], ko[a:b].view(torch.int32)), "keys_out != keys_in[vals_out]"
        sk = ko[a:b].view(torch.int32).to(torch.int64) & 0xFFFFFFFF
        ok = (sk[:-1] < sk[1:]) | ((sk[:-1] == sk[1:]) & (idx[:-1] < idx[1:]))
        assert bool(ok.all()), f"order/stability violated near {a}"
        del idx, sk, ok


@pytest.mark.parametrize("exchange", ["grouped", "fused"])
def test_distributed_fullsize_world1(exchange):
    """The distributed driver at the BASELINE size (2^28 u32/u32 AND-2, a process group of
    one): partition (or fused partition into the receive window), exchange, grouped local
    sort -- checked with the O(n) stable-sort certificate in a fresh process."""
    import os
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    code = r"""
import os, socket, torch, torch.distributed as dist
with socket.socket() as s:
    s.bind(("127.0.0.1", 0)); port = s.getsockname()[1]
os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
dist.init_process_group("gloo", rank=0, world_size=1)
import importlib.util, gen
spec = importlib.util.spec_from_file_location("fs", "tests/test_gpu_fullsize.py")
m = importlib.util.module_from_spec(spec); spec.loader.exec_module(m)
from paper_1611_01137_b200 import dist as hdist
n = 1 << 28
k = gen.keys(n, 32, "and2", device="cuda:0")
v = gen.values(n, 32, "index", device="cuda:0")
s = hdist.DistributedSorter(k, v, exchange="%s")
for _ in range(2):
    ko, vo, off = s.step()
torch.cuda.synchronize()
assert off == 0 and ko.numel() == n
m.certificate(k, ko, vo, 0, 32)
print("dist fullsize ok")
""" % exchange
    r = subprocess.run([sys.executable, "-c", code], cwd=root, env=dict(os.environ, PYTHONPATH=root),
                       capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-4000:]
    assert "dist fullsize ok" in r.stdout
