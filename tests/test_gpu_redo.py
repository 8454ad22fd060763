"""GPU parity of the redo paths of the fast rank (HRS_FLAG_FORCE_REDO).

The fast in-warp rank of k_scatter and k_local takes the order in which returning
shared-memory atomics serve the lanes of one instruction as the lanes' order; B200 serves
them in lane order, but PTX does not promise it.  Every caller therefore checks the order
it produced (the complete stability condition) and, when it is not the stable one, redoes
the tile / bucket with the rank that is stable by construction.  On this hardware that
branch never runs by itself, so these tests force every check to fail (tuning flag
HRS_FLAG_FORCE_REDO, or the HRS_FORCE_REDO=1 environment variable for entry points that
take no tuning) and compare the result with the oracle element by element, as the
ordinary parity tests do.  hrs_stats.redo_blocks proves the branch ran.

The redo path is the stable-by-construction LSD / partition of P:293-311 in the paper's
order; stability itself is reading #1 of DESIGN.md (BJ north_star)."""
import os
import subprocess
import sys

import numpy as np
import pytest
import torch

import gen
import oracle

pytestmark = pytest.mark.gpu
DEV = "cuda:0"
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
TYPES = [(32, 0), (32, 32), (32, 64), (64, 0), (64, 32), (64, 64)]
FORCE = 1  # HRS_FLAG_FORCE_REDO


def _np(t):
    return oracle._u64(t.cpu())


def _forced_sort(k, v, b, e, tuning=None):
    import paper_1611_01137_b200 as hrs
    t = dict(tuning or {})
    t["flags"] = FORCE
    kd = k.to(DEV)
    vd = v.to(DEV) if v is not None else None
    kb, vb = kd.element_size(), (vd.element_size() if vd is not None else 0)
    temp = torch.empty(hrs.temp_bytes(kd.numel(), kb, vb, b, e, t), dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort(kd, vd, b, e, tuning=t, temp=temp)
    st = hrs.get_stats(temp)
    ek, ev = oracle.sort(k, v, b, e)
    assert np.array_equal(_np(ko), ek), f"keys differ under forced redo (n={k.numel()}, [{b},{e}))"
    if v is not None:
        assert np.array_equal(_np(vo), ev), f"values differ under forced redo (n={k.numel()}, [{b},{e}))"
    return st


@pytest.mark.parametrize("kbits,vbits", TYPES)
@pytest.mark.parametrize("dist", ["uniform", "and2", "and4", "const"])
def test_forced_redo_default_tuning(kbits, vbits, dist):
    """Default thresholds: the scatter tiles of every counting pass redo (and the local
    sorts that take k_local: small classes, hand-offs, the wide variants)."""
    n = 300001
    k = gen.keys(n, kbits, dist, seed=13)
    v = gen.values(n, vbits, "random", seed=13) if vbits else None
    st = _forced_sort(k, v, 0, kbits)
    assert st["overflow"] == 0
    if dist in ("uniform", "and2"):
        # (constant / AND-4 digits make every warp take the exact rank, which needs no check)
        assert st["redo_blocks"] > 0, "the forced redo branch did not run"


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (32, 0), (64, 64), (64, 32)])
@pytest.mark.parametrize("tuning", [dict(local_threshold=300, merge_threshold=100, keys_per_tile=128),
                                    dict(local_threshold=64, merge_threshold=40, keys_per_tile=32),
                                    dict(local_threshold=2048, merge_threshold=1, keys_per_tile=512,
                                         local_classes=1)])
@pytest.mark.parametrize("dist", ["uniform", "and3"])
def test_forced_redo_local_paths(kbits, vbits, tuning, dist):
    """Small thresholds put every bucket in k_local (composite path for 32-bit keys and
    64-bit keys with <= 19 sort bits, pair path for wider 64-bit entries), and the
    single-configuration ablation routes everything through one class: all of them
    redo their LSD passes with the exact rank."""
    n = 60013
    k = gen.keys(n, kbits, dist, seed=17)
    v = gen.values(n, vbits, "index") if vbits else None
    st = _forced_sort(k, v, 0, kbits, tuning)
    assert st["redo_blocks"] > 0


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (64, 64)])
def test_forced_redo_bit_ranges(kbits, vbits):
    k = gen.keys(70001, kbits, "and2", seed=19)
    v = gen.values(70001, vbits, "random", seed=19)
    for b, e in ((0, 1), (3, 29), (8, 16), (1, kbits), (0, kbits - 3)):
        _forced_sort(k, v, b, e)
        _forced_sort(k, v, b, e, dict(local_threshold=100, merge_threshold=30, keys_per_tile=64))


def test_forced_redo_env_typed_and_fullsize():
    """HRS_FORCE_REDO=1 (read once at library load) in a fresh process: signed / float keys
    (hrs_sort_typed takes no tuning) and one 2^28 u32/u32 AND-3 sort in bench.py's launch
    configuration, checked with the O(n) stable-sort certificate."""
    code = r"""
import numpy as np, torch, gen, oracle
import paper_1611_01137_b200 as hrs
import importlib.util
_spec = importlib.util.spec_from_file_location("fullsize", "tests/test_gpu_fullsize.py")
_m = importlib.util.module_from_spec(_spec); _spec.loader.exec_module(_m)
certificate = _m.certificate
DEV = "cuda:0"
for dtype, kind in ((torch.int32, "int"), (torch.float64, "float")):
    kb = 32 if dtype == torch.int32 else 64
    k = gen.keys(100003, kb, "uniform", seed=3).view(dtype)
    v = gen.values(100003, 32, "index")
    ko, vo = hrs.sort(k.to(DEV), v.to(DEV))
    ek, ev = oracle.sort_typed(k.numpy(), oracle._u64(v), kind)
    ub = np.uint32 if kb == 32 else np.uint64
    assert np.array_equal(ko.cpu().numpy().view(ub), ek.view(ub)), dtype
    assert np.array_equal(oracle._u64(vo.cpu()), ev), dtype
n = 1 << 28
k = gen.keys(n, 32, "and3", device=DEV)
v = gen.values(n, 32, "index", device=DEV)
temp = torch.empty(hrs.temp_bytes(n, 4, 4), dtype=torch.uint8, device=DEV)
ko, vo = hrs.sort(k, v, temp=temp)
st = hrs.get_stats(temp)
certificate(k, ko, vo, 0, 32)
assert st["redo_blocks"] > 0 and st["overflow"] == 0, st
print("forced redo ok", st["redo_blocks"])
"""
    env = dict(os.environ, HRS_FORCE_REDO="1", PYTHONPATH=ROOT)
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, env=env, capture_output=True, text=True,
                       timeout=900)
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-4000:]
    assert "forced redo ok" in r.stdout


def test_unforced_run_reports_redo_count():
    """Without the flag the check still runs; on B200 the atomics serve lanes in order,
    so no block redoes (recorded, not required: a redo would still be correct)."""
    import paper_1611_01137_b200 as hrs
    n = 1 << 21
    k = gen.keys(n, 32, "uniform", seed=23, device=DEV)
    v = gen.values(n, 32, "index", device=DEV)
    temp = torch.empty(hrs.temp_bytes(n, 4, 4), dtype=torch.uint8, device=DEV)
    hrs.sort(k, v, temp=temp)
    st = hrs.get_stats(temp)
    assert st["redo_blocks"] >= 0
    print("unforced redo_blocks:", st["redo_blocks"])
