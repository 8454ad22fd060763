"""GPU parity: the CUDA path through the C ABI against the CPU oracle, element by element.

All integer work, so the bar is bit-exact keys and values (BJ north_star).  Inputs are
seeded synthetic workloads from gen/ (uniform and AND-m skew)."""
import os

import numpy as np
import pytest
import torch

import gen
import oracle
from oracle import plan

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

DEV = "cuda:0"
TYPES = [(32, 0), (32, 32), (32, 64), (64, 0), (64, 32), (64, 64)]


def _np(t: torch.Tensor) -> np.ndarray:
    return oracle._u64(t.cpu())


def _inputs(n, kbits, vbits, dist, seed, vkind="random"):
    k = gen.keys(n, kbits, dist, seed=seed)
    v = gen.values(n, vbits, vkind, seed=seed) if vbits else None
    return k, v


def _run_and_check(k, v, b, e, tuning=None, stats_expect=None):
    import paper_1611_01137_b200 as hrs
    kd = k.to(DEV)
    vd = v.to(DEV) if v is not None else None
    ko, vo = hrs.sort(kd, vd, b, e, tuning=tuning)
    torch.cuda.synchronize()
    ek, ev = oracle.sort(k, v, b, e)
    got_k = _np(ko)
    assert np.array_equal(got_k, ek), f"keys differ (n={k.numel()}, bits=[{b},{e}))"
    if v is not None:
        assert np.array_equal(_np(vo), ev), f"values differ (n={k.numel()}, bits=[{b},{e}))"
    return ko, vo


@pytest.mark.parametrize("kbits,vbits", TYPES)
@pytest.mark.parametrize("n", [0, 1, 2, 31, 32, 33, 1000, 4095, 4096, 4097, 8192, 8193, 12289, 100003])
def test_sizes_uniform(kbits, vbits, n):
    k, v = _inputs(n, kbits, vbits, "uniform", seed=n + 1)
    _run_and_check(k, v, 0, kbits)


@pytest.mark.parametrize("kbits,vbits", TYPES)
@pytest.mark.parametrize("dist", ["and2", "and3", "and4", "const"])
def test_skewed(kbits, vbits, dist):
    k, v = _inputs(300001, kbits, vbits, dist, seed=7)
    _run_and_check(k, v, 0, kbits)


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (64, 64), (64, 0)])
def test_one_million_and_odd_values(kbits, vbits):
    for dist in ("uniform", "and3"):
        k, v = _inputs((1 << 20) + 17, kbits, vbits, dist, seed=3)
        _run_and_check(k, v, 0, kbits)


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (64, 32)])
def test_bit_ranges(kbits, vbits):
    k, v = _inputs(50000, kbits, vbits, "and2", seed=4)
    ranges = [(0, 1), (7, 9), (3, 29), (8, 16), (kbits - 1, kbits), (5, 5), (0, 8), (1, kbits), (0, kbits - 3)]
    if kbits == 64:
        ranges += [(0, 33), (17, 61), (32, 64), (56, 64)]
    for b, e in ranges:
        _run_and_check(k, v, b, e)


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (32, 0), (64, 64)])
def test_partial_ranges_deep_buckets(kbits, vbits):
    """begin = 0 with end < key bits at a size where local sorts run after two counting
    passes: the key bits above end_bit vary inside a bucket and must be carried (not
    rebuilt from the bucket's common bits)."""
    k, v = _inputs((1 << 22) + 5, kbits, vbits, "uniform", seed=21)
    for b, e in ((0, kbits - 3), (0, 24), (0, 20), (2, kbits - 1)):
        _run_and_check(k, v, b, e)


def test_tie_heavy_stability():
    """Constant and two-valued keys: only stability decides the value order."""
    n = 200000
    for keys in (torch.zeros(n, dtype=torch.int32).view(torch.uint32),
                 (torch.arange(n, dtype=torch.int32) % 2).view(torch.uint32),
                 torch.full((n,), -1, dtype=torch.int32).view(torch.uint32),
                 torch.full((n,), 0x5A5A5A5A, dtype=torch.int32).view(torch.uint32)):
        v = gen.values(n, 32, "index")
        _run_and_check(keys, v, 0, 32)


def test_sorted_and_reverse_inputs():
    n = 123457
    k = gen.keys(n, 32, "uniform", seed=2)
    ks, _ = oracle.sort(k, None, 0, 32)
    ks_t = torch.from_numpy(ks.astype(np.uint32).view(np.int32)).view(torch.uint32)
    _run_and_check(ks_t, gen.values(n, 32, "index"), 0, 32)
    _run_and_check(ks_t.view(torch.int32).flip(0).contiguous().view(torch.uint32), gen.values(n, 32, "index"), 0, 32)


# ------------------------------------------------------------- deep recursion via tuning overrides

TUNINGS = [
    dict(local_threshold=64, merge_threshold=40, keys_per_tile=32),
    dict(local_threshold=300, merge_threshold=100, keys_per_tile=128),
    dict(local_threshold=3, merge_threshold=2, keys_per_tile=4),
    dict(local_threshold=200, merge_threshold=1, keys_per_tile=1),
    dict(local_threshold=4096, merge_threshold=4096, keys_per_tile=3072),
]


@pytest.mark.parametrize("tuning", TUNINGS)
@pytest.mark.parametrize("dist", ["uniform", "and2", "and4", "const"])
@pytest.mark.parametrize("kbits,vbits", [(32, 32), (64, 64)])
def test_threshold_overrides_and_structure(tuning, dist, kbits, vbits):
    """Forcing tiny thresholds exercises deep recursion, merging, every size class and
    last-digit exhaustion; the pass/bucket/local structure must equal the paper-order
    MSD simulation (oracle/plan.py) exactly."""
    import paper_1611_01137_b200 as hrs
    n = 5000
    k, v = _inputs(n, kbits, vbits, dist, seed=11)
    kd, vd = k.to(DEV), v.to(DEV)
    tb = hrs.temp_bytes(n, kbits // 8, vbits // 8, 0, kbits, tuning)
    temp = torch.empty(tb, dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort(kd, vd, 0, kbits, tuning=tuning, temp=temp)
    st = hrs.get_stats(temp)
    ek, ev = oracle.sort(k, v, 0, kbits)
    assert np.array_equal(_np(ko), ek) and np.array_equal(_np(vo), ev)
    # the library's own size-class table (hrs_class_capacity) labels the oracle's entries:
    # the class boundaries are a tuning of this build (reading #20), not part of the method
    sim = plan.simulate_msd(oracle._u64(k), None, 0, kbits, tuning["local_threshold"],
                            tuning["merge_threshold"], tuning["keys_per_tile"],
                            class_capacities=tuple(hrs.class_capacities()))
    assert st["overflow"] == 0
    assert st["counting_passes"] == sim.counting_passes
    assert st["recs_in_pass"] == sim.recs_in_pass
    assert st["tiles_in_pass"] == sim.tiles_in_pass
    assert st["buckets_in_pass"] == sim.buckets_in_pass
    assert st["local_buckets"] == sim.local_buckets
    assert st["local_recs"] == sim.local_recs
    assert st["merged_groups"] == sim.merged_groups
    assert st["skipped_recs_in_pass"] == sim.skipped_in_pass
    per_class = [0] * 8
    for e in sim.local_entries:
        per_class[e[3]] += 1
    assert st["local_in_class"] == per_class
    assert st["bytes_min"] == plan.bytes_min(sim, kbits // 8, vbits // 8)


def test_single_local_config_ablation():
    n = 40000
    k, v = _inputs(n, 32, 32, "and2", seed=12)
    _run_and_check(k, v, 0, 32, tuning=dict(local_threshold=2048, merge_threshold=1, keys_per_tile=512,
                                            local_classes=1))


def test_table2_worked_example_on_gpu():
    """Table 2 with keys (a << 8) | b, ∂ˆ = 3, no merging, KPB = 4."""
    import paper_1611_01137_b200 as hrs
    toks = "31 12 01 23 12 22 12 00 11 10 10 31 03 13 12 03".split()
    final = "00 01 03 03 10 10 11 12 12 12 12 13 22 23 31 31".split()
    enc = [(int(t[0]) << 8) | int(t[1]) for t in toks]
    k = torch.tensor(enc, dtype=torch.int32).view(torch.uint32).to(DEV)
    v = torch.arange(16, dtype=torch.int32).view(torch.uint32).to(DEV)
    tun = dict(local_threshold=3, merge_threshold=1, keys_per_tile=4)
    temp = torch.empty(hrs.temp_bytes(16, 4, 4, 0, 16, tun), dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort(k, v, 0, 16, tuning=tun, temp=temp)
    assert ko.view(torch.int32).cpu().tolist() == [(int(t[0]) << 8) | int(t[1]) for t in final]
    assert vo.view(torch.int32).cpu().tolist() == [7, 2, 12, 15, 9, 10, 8, 1, 4, 6, 14, 13, 5, 3, 0, 11]
    st = hrs.get_stats(temp)
    assert st["counting_passes"] == 2 and st["recs_in_pass"] == [16, 12] and st["local_buckets"] == 2
    # pass 1 alone: the partition building block reproduces Table 2 row 5 and the offsets
    k1, v1, offs = hrs.partition_pass(k, v, 8, 16)
    assert v1.view(torch.int32).cpu().tolist() == [2, 7, 12, 15, 1, 4, 6, 8, 9, 10, 13, 14, 3, 5, 0, 11]
    assert offs.view(torch.int64).cpu().tolist()[:5] == [0, 4, 12, 14, 16]
    h = hrs.digit_histogram(k, 8, 16)
    assert h.view(torch.int64).cpu().tolist()[:4] == [4, 8, 2, 2]


# ------------------------------------------------------------- building blocks

@pytest.mark.parametrize("kbits", [32, 64])
@pytest.mark.parametrize("n", [0, 1, 4097, 1000003])
def test_digit_histogram(kbits, n):
    import paper_1611_01137_b200 as hrs
    k = gen.keys(n, kbits, "and2", seed=5)
    kd = k.to(DEV)
    for lo, hi in ((kbits - 8, kbits), (0, 8), (3, 7), (kbits - 1, kbits)):
        h = hrs.digit_histogram(kd, lo, hi)
        exp = oracle.histogram(k, lo, hi)
        assert np.array_equal(_np(h), exp), (lo, hi)


@pytest.mark.parametrize("kbits,vbits", TYPES)
def test_partition_pass(kbits, vbits):
    import paper_1611_01137_b200 as hrs
    for n in (1, 4097, 654321):
        k, v = _inputs(n, kbits, vbits, "and3", seed=n)
        kd = k.to(DEV)
        vd = v.to(DEV) if v is not None else None
        for lo, hi in ((kbits - 8, kbits), (5, 11)):
            ko, vo, offs = hrs.partition_pass(kd, vd, lo, hi)
            ek, ev, eo = oracle.partition_pass(k, v, lo, hi)
            assert np.array_equal(_np(ko), ek)
            if v is not None:
                assert np.array_equal(_np(vo), ev)
            assert np.array_equal(_np(offs), eo)


# ------------------------------------------------------------- properties

def test_deterministic_repeats():
    import paper_1611_01137_b200 as hrs
    n = 1 << 21
    k = gen.keys(n, 32, "and3", seed=9, device=DEV)
    v = gen.values(n, 32, "index", device=DEV)
    ref = None
    for _ in range(5):
        ko, vo = hrs.sort(k, v)
        cur = (ko.clone(), vo.clone())
        if ref is None:
            ref = cur
        else:
            assert torch.equal(cur[0].view(torch.int32), ref[0].view(torch.int32))
            assert torch.equal(cur[1].view(torch.int32), ref[1].view(torch.int32))


def test_errors_on_gpu():
    import paper_1611_01137_b200 as hrs
    k = torch.zeros(100, dtype=torch.uint32, device=DEV)
    with pytest.raises(hrs.HrsError):
        hrs.sort(k, None, 0, 33)
    # aliasing: output overlapping input
    with pytest.raises(hrs.HrsError, match="ALIASING"):
        hrs.sort(k, None, keys_out=k)
    # misaligned u32 pointer (view starting one byte in)
    raw = torch.zeros(404, dtype=torch.uint8, device=DEV)
    with pytest.raises(hrs.HrsError):
        import ctypes
        sz = ctypes.c_size_t(1 << 20)
        t = torch.empty(1 << 20, dtype=torch.uint8, device=DEV)
        hrs.check(hrs.lib.hrs_sort_ex(ctypes.c_void_p(t.data_ptr()), ctypes.byref(sz),
                                      ctypes.c_void_p(raw.data_ptr() + 1), ctypes.c_void_p(raw.data_ptr() + 404),
                                      None, None, 10, 4, 0, 0, 32, None, None), "misaligned")


@pytest.mark.parametrize("kbits,vbits", [(32, 32), (32, 64), (32, 0), (64, 32)])
@pytest.mark.parametrize("dist_name", ["uniform", "and2"])
def test_counting_local_sort_paths(kbits, vbits, dist_name):
    """2^20 records: one counting pass leaves ~4096-record buckets, so the counting local
    sort (k_local_cnt) runs -- with key reconstruction ([0, 32) of u32 keys), without it
    (begin > 0: tie fix-up on gathered low key bits; end < 32: carried upper bits), and
    with AND-2 keys whose 4-bit counters overflow (hand-off to k_local)."""
    k, v = _inputs((1 << 20) + 3, kbits, vbits, dist_name, seed=31)
    for b, e in ((0, kbits), (2, kbits), (0, kbits - 1), (5, kbits - 2)):
        _run_and_check(k, v, b, e)


def test_graph_replay_follows_new_data():
    """Small sorts replay a captured CUDA graph from the second identical call on: the
    replays must sort whatever the buffers hold now (new data every call), for several
    sizes and with HRS_GRAPHS' cache keyed on every argument."""
    import paper_1611_01137_b200 as hrs
    for n, kbits, vbits in ((70001, 32, 32), (1 << 20, 32, 0), (300000, 64, 64)):
        kd = torch.empty(n, dtype=torch.uint32 if kbits == 32 else torch.uint64, device=DEV)
        vd = torch.empty(n, dtype=torch.uint32 if vbits == 32 else torch.uint64, device=DEV) if vbits else None
        ko, vo = torch.empty_like(kd), (torch.empty_like(vd) if vbits else None)
        temp = torch.empty(hrs.temp_bytes(n, kbits // 8, vbits // 8), dtype=torch.uint8, device=DEV)
        l0 = hrs.launch_count()
        for i, dist in enumerate(("uniform", "and3", "uniform", "and2")):
            k, v = _inputs(n, kbits, vbits, dist, seed=100 + i)
            kd.copy_(k.to(DEV))
            if vbits:
                vd.copy_(v.to(DEV))
            hrs.sort(kd, vd, keys_out=ko, values_out=vo, temp=temp)
            torch.cuda.synchronize()
            ek, ev = oracle.sort(k, v, 0, kbits)
            assert np.array_equal(_np(ko), ek), (n, i)
            if vbits:
                assert np.array_equal(_np(vo), ev), (n, i)
        assert hrs.launch_count() - l0 >= 4 * 10  # replays still count their kernels


@pytest.mark.parametrize("dtype,vbits", [(torch.int32, 32), (torch.int64, 64), (torch.float32, 32),
                                         (torch.float64, 0), (torch.float32, 64)])
@pytest.mark.parametrize("n", [1, 1000, 70001, (1 << 20) + 9])
def test_typed_keys(dtype, vbits, n):
    """Signed and IEEE-754 keys (hrs_sort_typed) against the oracle's
    plain definition of their order: random bit patterns (so NaNs with every payload,
    ±inf, ±0, denormals and int min/max occur) plus AND-3 skew, bit-exact keys and values."""
    import paper_1611_01137_b200 as hrs
    kb = 32 if dtype in (torch.int32, torch.float32) else 64
    kind = "int" if dtype in (torch.int32, torch.int64) else "float"
    for dist in ("uniform", "and3", "const"):
        bits = gen.keys(n, kb, dist, seed=41)
        k = bits.view(dtype)
        v = gen.values(n, vbits, "index") if vbits else None
        ko, vo = hrs.sort(k.to(DEV), v.to(DEV) if vbits else None)
        torch.cuda.synchronize()
        kn = k.numpy() if dtype != torch.int32 else k.numpy()
        ek, ev = oracle.sort_typed(kn, None if v is None else oracle._u64(v), kind)
        ub = np.uint32 if kb == 32 else np.uint64
        assert np.array_equal(ko.cpu().numpy().view(ub), ek.view(ub)), (dtype, n, dist)
        if vbits:
            assert np.array_equal(oracle._u64(vo.cpu()), ev), (dtype, n, dist)


@pytest.mark.parametrize("kbits,vbits", [(64, 0), (64, 32), (64, 64)])
@pytest.mark.parametrize("n", [786431, (1 << 20) + 5, 1572869])
def test_wide_configurations_64bit(kbits, vbits, n):
    """One counting pass leaves 256 buckets of ~n/256 records with 56 sort bits, which
    the 64-bit local sort hands to the wide variant: mean 3072 / 4096 / 6144 records put
    them in the wide lists of size class 5 (<= 4096), 6 (<= 4608) and the largest."""
    for dist in ("uniform", "and2"):
        k, v = _inputs(n, kbits, vbits, dist, seed=n % 1000 + kbits + vbits)
        _run_and_check(k, v, 0, kbits)


# ------------------------------------------------------------- the named §8(b) entry points

@pytest.mark.parametrize("name,kbits,vbits", [("hrs_sort_keys_u32", 32, 0), ("hrs_sort_keys_u64", 64, 0),
                                              ("hrs_sort_pairs_u32_u32", 32, 32),
                                              ("hrs_sort_pairs_u32_u64", 32, 64),
                                              ("hrs_sort_pairs_u64_u32", 64, 32),
                                              ("hrs_sort_pairs_u64_u64", 64, 64)])
def test_named_entry_points(name, kbits, vbits):
    """Each typed C entry point of include/hrs.h called directly through ctypes (two-phase
    temp protocol, raw device pointers, the current stream), against the oracle."""
    import ctypes
    import paper_1611_01137_b200 as hrs
    fn = getattr(hrs.lib, name)
    for n, dist, (b, e) in ((100003, "and2", (0, kbits)), (4097, "uniform", (3, kbits - 2)), (0, "uniform", (0, kbits)),
                            (1 << 20, "uniform", (0, kbits))):
        k, v = _inputs(n, kbits, vbits, dist, seed=n + 5)
        kd = k.to(DEV)
        ko = torch.empty_like(kd)
        vd = v.to(DEV) if v is not None else None
        vo = torch.empty_like(vd) if v is not None else None
        P = ctypes.c_void_p
        ptr = lambda t: P(t.data_ptr()) if t is not None and t.numel() else P(0)  # noqa: E731
        data = [ptr(kd), ptr(ko)] + ([ptr(vd), ptr(vo)] if vbits else [])
        sz = ctypes.c_size_t(0)
        hrs.check(fn(None, ctypes.byref(sz), *data, n, b, e, None), name + "(size)")
        temp = torch.empty(max(sz.value, 256), dtype=torch.uint8, device=DEV)
        sz = ctypes.c_size_t(temp.numel())
        stream = P(torch.cuda.current_stream().cuda_stream)
        hrs.check(fn(P(temp.data_ptr()), ctypes.byref(sz), *data, n, b, e, stream), name)
        torch.cuda.synchronize()
        ek, ev = oracle.sort(k, v, b, e)
        assert np.array_equal(_np(ko), ek), (name, n)
        if vbits:
            assert np.array_equal(_np(vo), ev), (name, n)


def test_binding_checks_outputs_and_streams():
    """The binding rejects short / mistyped output buffers (the library writes n elements
    through raw pointers) and typed keys in partition_pass; a sort on a side stream with
    binding-allocated temp gives the oracle's result."""
    import paper_1611_01137_b200 as hrs
    k = gen.keys(5000, 32, "uniform", seed=1).to(DEV)
    with pytest.raises(ValueError):
        hrs.sort(k, None, keys_out=torch.empty(4999, dtype=torch.uint32, device=DEV))
    with pytest.raises(ValueError):
        hrs.sort(k, k.clone(), values_out=torch.empty(5000, dtype=torch.uint64, device=DEV))
    with pytest.raises(TypeError):
        hrs.partition_pass(k.view(torch.int32), None, 24, 32)
    s = torch.cuda.Stream()
    kk, vv = _inputs(1 << 20, 32, 32, "and2", seed=3)
    kd, vd = kk.to(DEV), vv.to(DEV)
    s.wait_stream(torch.cuda.current_stream())
    ko, vo = hrs.sort(kd, vd, stream=s)
    s.synchronize()
    ek, ev = oracle.sort(kk, vv, 0, 32)
    assert np.array_equal(_np(ko), ek) and np.array_equal(_np(vo), ev)


# ------------------------------------------------------------- grouped input (first pass given)

@pytest.mark.parametrize("kbits,vbits", TYPES)
@pytest.mark.parametrize("dist", ["uniform", "and3", "const"])
def test_sort_grouped(kbits, vbits, dist):
    """hrs_sort_grouped: an input stably partitioned on its first digit (the oracle's pass,
    P:503-509) with that digit's histogram; the library starts at the second digit.  A
    stable partition followed by the stable sort of the rest is the stable sort of the
    original input, so the result must equal the oracle's sort of the ungrouped data;
    bit ranges with a narrow first digit and tiny thresholds (deep recursion) included."""
    import paper_1611_01137_b200 as hrs
    for n, (b, e), tun in ((300001, (0, kbits), None), (70001, (3, kbits - 4), None),
                           (20011, (0, kbits), dict(local_threshold=64, merge_threshold=40, keys_per_tile=32)),
                           (5000, (0, 5), None), (100003, (kbits - 8, kbits), None), (9000, (0, 12), None)):
        k, v = _inputs(n, kbits, vbits, dist, seed=n)
        lo, hi = max(b, e - 8), e
        gk, gv, offs = oracle.partition_pass(k, v, lo, hi)
        hist = np.diff(offs.astype(np.int64))
        tk = torch.from_numpy(gk.astype(np.uint64).view(np.int64)).to(DEV)
        tk = tk.view(torch.uint64) if kbits == 64 else tk.to(torch.int32).view(torch.uint32)
        tv = None
        if v is not None:
            tv = torch.from_numpy(gv.astype(np.uint64).view(np.int64)).to(DEV)
            tv = tv.view(torch.uint64) if vbits == 64 else tv.to(torch.int32).view(torch.uint32)
        ko, vo = hrs.sort_grouped(tk, tv, hist.tolist(), b, e, tuning=tun)
        torch.cuda.synchronize()
        ek, ev = oracle.sort(k, v, b, e)
        assert np.array_equal(_np(ko), ek), (n, b, e, tun)
        if v is not None:
            assert np.array_equal(_np(vo), ev), (n, b, e, tun)


def test_sort_grouped_stats_skip_first_pass():
    """The first pass moves nothing: bytes_min drops by R(K + 2(K+V)) for that pass."""
    import paper_1611_01137_b200 as hrs
    n = 1 << 22
    k = gen.keys(n, 32, "uniform", seed=7)
    v = gen.values(n, 32, "index")
    gk, gv, offs = oracle.partition_pass(k, v, 24, 32)
    tk = torch.from_numpy(gk.astype(np.int64)).to(torch.int32).view(torch.uint32).to(DEV)
    tv = torch.from_numpy(gv.astype(np.int64)).to(torch.int32).view(torch.uint32).to(DEV)
    temp = torch.empty(hrs.temp_bytes(n, 4, 4), dtype=torch.uint8, device=DEV)
    ko, vo = hrs.sort_grouped(tk, tv, np.diff(offs.astype(np.int64)).tolist(), temp=temp)
    st = hrs.get_stats(temp)
    full = plan.simulate_msd(oracle._u64(k), None, 0, 32, 8192, 2048, hrs.max_keys_per_tile(4, 4))
    assert st["recs_in_pass"][0] == 0 and st["recs_in_pass"][1:] == full.recs_in_pass[1:]
    assert st["bytes_min"] == plan.bytes_min(full, 4, 4) - n * (4 + 2 * 8)
    ek, ev = oracle.sort(k, v, 0, 32)
    assert np.array_equal(_np(ko), ek) and np.array_equal(_np(vo), ev)


def test_copy_pieces():
    """hrs_copy_pieces (the distributed sort's own pieces): random pieces against numpy."""
    import paper_1611_01137_b200 as hrs
    rng = np.random.default_rng(5)
    for dt in (torch.int32, torch.int64):
        src = torch.arange(300000, dtype=dt, device=DEV)
        dst = torch.full((300000,), -1, dtype=dt, device=DEV)
        cuts = np.sort(rng.choice(np.arange(1, 300000), 40, replace=False))
        lens = np.diff(np.concatenate([[0], cuts, [300000]]))
        perm = rng.permutation(len(lens))
        soffs = np.concatenate([[0], np.cumsum(lens)[:-1]])
        pieces, d = [], 0
        for i in perm:
            pieces.append((int(soffs[i]), d, int(lens[i])))
            d += int(lens[i])
        hrs.copy_pieces(dst, src, pieces + [(0, 0, 0)])
        exp = np.concatenate([np.arange(soffs[i], soffs[i] + lens[i]) for i in perm])
        assert np.array_equal(dst.cpu().numpy(), exp)


@pytest.mark.parametrize("kbits,vbits", TYPES)
def test_leading_constant_digits_skip(kbits, vbits):
    """Reading #22: buckets still in the input whose digit is constant are not scattered.
    Constant keys, 64-bit keys below 2^32 (four leading constant digits), keys with a
    constant top byte, and a constant second digit after a real pass (no skip): output
    against the oracle, structure (skipped records per pass) against the MSD simulation."""
    import paper_1611_01137_b200 as hrs
    n = 200003
    base = gen.keys(n, kbits, "uniform", seed=8)
    bo = oracle._u64(base)
    cases = [np.full(n, 0x5A5A5A5A5A5A5A5A if kbits == 64 else 0x5A5A5A5A, dtype=np.uint64),
             bo & np.uint64(0x00FFFFFF if kbits == 32 else 0xFFFFFFFF),
             (bo & np.uint64((1 << (kbits - 8)) - 1)) | np.uint64(0xC3 << (kbits - 8)),
             (bo & ~np.uint64(0xFF << (kbits - 16))) | np.uint64(0x5 << (kbits - 16))]
    tun = dict(local_threshold=2048, merge_threshold=512, keys_per_tile=1024)
    for kk in cases:
        k = torch.from_numpy(kk.view(np.int64).copy())
        k = k.view(torch.uint64) if kbits == 64 else k.to(torch.int32).view(torch.uint32)
        v = gen.values(n, vbits, "random", seed=9) if vbits else None
        for t in (None, tun):
            kd, vd = k.to(DEV), (v.to(DEV) if v is not None else None)
            temp = torch.empty(hrs.temp_bytes(n, kbits // 8, vbits // 8, 0, kbits, t), dtype=torch.uint8, device=DEV)
            ko, vo = hrs.sort(kd, vd, tuning=t, temp=temp)
            st = hrs.get_stats(temp)
            ek, ev = oracle.sort(k, v, 0, kbits)
            assert np.array_equal(_np(ko), ek)
            if v is not None:
                assert np.array_equal(_np(vo), ev)
            dt = t or hrs.default_tuning(kbits // 8, vbits // 8)
            sim = plan.simulate_msd(kk, None, 0, kbits, dt["local_threshold"], dt["merge_threshold"],
                                    dt["keys_per_tile"])
            assert st["skipped_recs_in_pass"] == sim.skipped_in_pass
            assert st["bytes_min"] == plan.bytes_min(sim, kbits // 8, vbits // 8)


# ------------------------------------------------------------- array-of-structs records

@pytest.mark.parametrize("kb,vb", [(4, 4), (4, 8), (8, 4), (8, 8), (4, 0), (8, 0)])
@pytest.mark.parametrize("key_first", [True, False])
def test_sort_records(kb, vb, key_first):
    """hrs_sort_records: interleaved records decomposed, sorted, recomposed.  Unsigned keys
    over a bit range and signed / float keys by value; the oracle sorts the (key, record
    index) pairs stably and the expected output is the records in that order."""
    import paper_1611_01137_b200 as hrs
    n = 100003
    rng = np.random.default_rng(kb * 10 + vb + key_first)
    raw = rng.integers(0, 256, size=(n, kb + vb), dtype=np.uint8)
    raw[: n // 3, :] = raw[n // 2: n // 2 + n // 3, :]  # duplicate records: ties
    koff = 0 if key_first else vb
    kdt = {4: np.uint32, 8: np.uint64}[kb]
    keys = np.ascontiguousarray(raw[:, koff:koff + kb]).view(kdt).reshape(-1)
    rd = torch.from_numpy(raw.copy()).to(DEV)
    for kind, (b, e) in (("uint", (0, 8 * kb)), ("uint", (3, 8 * kb - 5)), ("int", (0, 8 * kb)), ("float", (0, 8 * kb))):
        out = hrs.sort_records(rd, kb, vb, key_first=key_first, kind=kind, begin_bit=b, end_bit=e)
        torch.cuda.synchronize()
        idx = np.arange(n, dtype=np.uint64)
        if kind == "uint":
            _, order = oracle.sort(keys, idx, b, e)
        else:
            tdt = {("int", 4): np.int32, ("int", 8): np.int64, ("float", 4): np.float32, ("float", 8): np.float64}
            _, order = oracle.sort_typed(keys.view(tdt[(kind, kb)]), idx, kind)
        exp = raw[order.astype(np.int64)]
        assert np.array_equal(out.cpu().numpy(), exp), (kind, b, e)


def test_conditional_graph_replays():
    """(run in a fresh process with HRS_GRAPH_COND=1: conditional capture is opt-in)"""
    import subprocess
    import sys
    code = ("import sys; sys.path.insert(0, 'tests'); import test_gpu_sort as t; "
            "t._conditional_graph_replays()")
    env = dict(os.environ, HRS_GRAPH_COND="1", PYTHONPATH=ROOT)
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, env=env, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-4000:]


def _conditional_graph_replays():
    """Small sorts replay a captured CUDA graph whose later passes and local-sort launches are
    conditional nodes set on the device: replays of inputs with different structure (one
    pass + local sorts, all passes for constant keys, deep AND-4 recursion with merging and
    hand-offs, tiny thresholds) through the same cached graph must all match the oracle."""
    import paper_1611_01137_b200 as hrs
    for n, kbits, vbits, tun in ((1 << 20, 32, 0, None), (200003, 64, 64, None), (150001, 32, 32,
                                 dict(local_threshold=300, merge_threshold=100, keys_per_tile=128))):
        kd = torch.empty(n, dtype=torch.uint32 if kbits == 32 else torch.uint64, device=DEV)
        vd = torch.empty(n, dtype=torch.uint32 if vbits == 32 else torch.uint64, device=DEV) if vbits else None
        ko, vo = torch.empty_like(kd), (torch.empty_like(vd) if vbits else None)
        temp = torch.empty(hrs.temp_bytes(n, kbits // 8, vbits // 8, 0, kbits, tun), dtype=torch.uint8, device=DEV)
        for i, dist in enumerate(("uniform", "uniform", "const", "and4", "uniform", "and2", "const", "and3")):
            k, v = _inputs(n, kbits, vbits, dist, seed=200 + i)
            kd.copy_(k.to(DEV))
            if vbits:
                vd.copy_(v.to(DEV))
            hrs.sort(kd, vd, keys_out=ko, values_out=vo, temp=temp, tuning=tun)
            torch.cuda.synchronize()
            ek, ev = oracle.sort(k, v, 0, kbits)
            assert np.array_equal(_np(ko), ek), (n, dist, i)
            if vbits:
                assert np.array_equal(_np(vo), ev), (n, dist, i)


@pytest.mark.parametrize("kbits,vbits", TYPES)
def test_partition_pass_to_windows(kbits, vbits):
    """hrs_partition_pass_to (the fused exchange's scatter): every digit's
    run goes to its own window at its own offset -- here three separate device buffers in a
    scrambled bucket order with gaps -- and must equal the oracle's stable partition."""
    import paper_1611_01137_b200 as hrs
    rng = np.random.default_rng(kbits + vbits)
    for n, dist, (lo, hi) in ((300001, "and2", (kbits - 8, kbits)), (70001, "uniform", (3, 9)), (1, "uniform", (0, 8))):
        k, v = _inputs(n, kbits, vbits, dist, seed=n)
        ek, ev, eo = oracle.partition_pass(k, v, lo, hi)
        r = 1 << (hi - lo)
        cnt = np.diff(eo.astype(np.int64))
        win = rng.integers(0, 3, size=r)
        order = rng.permutation(r)
        sizes, offs = [0, 0, 0], [0] * r
        for d in order:  # place the runs window by window in a scrambled order, with gaps
            offs[d] = (int(win[d]) << 48) | (sizes[win[d]] + 7)
            sizes[win[d]] += int(cnt[d]) + 7
        kd = k.to(DEV)
        vd = v.to(DEV) if v is not None else None
        kwin = [torch.zeros(sz + 8, dtype=kd.dtype, device=DEV) for sz in sizes]
        vwin = [torch.zeros(sz + 8, dtype=vd.dtype, device=DEV) for sz in sizes] if v is not None else None
        hrs.partition_pass_to(kd, vd, lo, hi, offs, kwin, vwin)
        torch.cuda.synchronize()
        for d in range(r):
            w, o, c = offs[d] >> 48, offs[d] & ((1 << 48) - 1), int(cnt[d])
            assert np.array_equal(_np(kwin[w][o:o + c]), ek[int(eo[d]):int(eo[d]) + c]), (n, d)
            if v is not None:
                assert np.array_equal(_np(vwin[w][o:o + c]), ev[int(eo[d]):int(eo[d]) + c]), (n, d)
