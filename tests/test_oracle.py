"""Pins for the CPU oracle (no GPU).  Each test checks the oracle against something
other than itself: the paper's printed worked example, brute force, a library
routine (numpy's stable argsort), or an invariant of the stable sort."""
import itertools
import os

import numpy as np
import pytest
import torch

import gen
import oracle
from oracle import plan

GOLDEN = os.path.join(os.path.dirname(__file__), "golden", "table2.txt")


def _golden():
    out = {}
    for line in open(GOLDEN, encoding="utf-8"):
        line = line.strip()
        if not line or line.startswith("#"):
            continue
        name, vals = line.split("=", 1)
        out[name.strip()] = vals.split()
    return out


def _b4(tokens):
    """Base-4 two-digit keys as printed in Table 2 -> 4-bit integers."""
    return np.array([int(t, 4) for t in tokens], dtype=np.uint64)


# ---------------------------------------------------------------- Table 2

def test_table2_counting_pass_matches_paper():
    g = _golden()
    keys = _b4(g["keys"])
    # d = 2: the most-significant digit of a 4-bit key is bits [2, 4)
    assert oracle.histogram(keys, 2, 4).tolist() == [int(x) for x in g["histogram"]]
    ko, _, offs = oracle.partition_pass(keys, None, 2, 4)
    assert offs[:4].tolist() == [int(x) for x in g["prefix_sum"]]
    assert ko.tolist() == _b4(g["pass1"]).tolist()
    # second-digit histograms of buckets 0 and 1
    assert oracle.histogram(ko[0:4], 0, 2).tolist() == [int(x) for x in g["bucket0_hist"]]
    assert oracle.histogram(ko[4:12], 0, 2).tolist() == [int(x) for x in g["bucket1_hist"]]
    _, _, o0 = oracle.partition_pass(ko[0:4], None, 0, 2)
    _, _, o1 = oracle.partition_pass(ko[4:12], None, 0, 2)
    assert o0[:4].tolist() == [int(x) for x in g["bucket0_pref"]]
    assert o1[:4].tolist() == [int(x) for x in g["bucket1_pref"]]


def test_table2_full_sort_matches_paper():
    g = _golden()
    keys = _b4(g["keys"])
    ko, vo = oracle.sort(keys, np.arange(16), 0, 4)
    assert ko.tolist() == _b4(g["final"]).tolist()


def test_table2_msd_structure_matches_paper():
    """The MSD bookkeeping with 8-bit digits on keys encoded as (a << 8) | b, ∂ˆ = 3,
    no merging: two counting passes, buckets 2 and 3 local-sorted."""
    g = _golden()
    enc = lambda toks: np.array([(int(t[0]) << 8) | int(t[1]) for t in toks], dtype=np.uint64)
    keys = enc(g["keys"])
    r = plan.simulate_msd(keys, np.arange(16), 0, 16, local_threshold=3, merge_threshold=1, keys_per_tile=4)
    assert r.keys.tolist() == enc(g["final"]).tolist()
    assert r.counting_passes == 2
    assert r.recs_in_pass == [16, 12]          # buckets 0 and 1 (4 + 8 keys) are re-partitioned
    assert r.buckets_in_pass == [1, 2]
    assert r.tiles_in_pass == [4, 1 + 2]
    assert [(e[0], e[1]) for e in r.local_entries] == [(12, 2), (14, 2)]   # buckets 2 and 3
    # and the stable result agrees with the LSD oracle on the same data
    ko, vo = oracle.sort(keys, np.arange(16), 0, 16)
    assert ko.tolist() == r.keys.tolist() and vo.tolist() == r.vals.tolist()


# ---------------------------------------------------------------- brute force

def _insertion_sort(recs, begin, end):
    """Stable by construction: an element moves left only past strictly greater keys."""
    w = end - begin
    sk = lambda x: (x >> begin) % (1 << w)  # noqa: E731  (different formulation from the oracle)
    out = []
    for r in recs:
        i = len(out)
        while i > 0 and sk(out[i - 1][0]) > sk(r[0]):
            i -= 1
        out.insert(i, r)
    return out


@pytest.mark.parametrize("shift,width,extra", [(0, 64, 0), (30, 32, 0), (62, 64, 0), (5, 64, 1)])
def test_brute_force_all_short_sequences(shift, width, extra):
    """Every sequence of length <= 5 over a 4-letter alphabet (plus length 6 for one
    embedding), symbols placed at bit `shift`, junk in the other bits, values = index."""
    rng = np.random.default_rng(shift)
    ranges = [(shift, shift + 2), (shift, shift + 1), (shift + 1, shift + 2), (shift, shift)]
    if shift + 2 < width:
        ranges.append((shift, width))
    maxlen = 6 if shift == 0 else 5
    for L in range(0, maxlen + 1):
        for seq in itertools.product(range(4), repeat=L):
            junk = [int(x) for x in rng.integers(0, 1 << 62, size=L, dtype=np.int64)]
            if extra == 0:
                junk = [j & ~(3 << shift) & ((1 << width) - 1) for j in junk]
            else:
                junk = [j & ~(3 << shift) & ((1 << width) - 1) & ~0xFFF for j in junk]
            keys = [(s << shift) | j for s, j in zip(seq, junk)]
            recs = list(zip(keys, range(L)))
            for b, e in ranges:
                exp = _insertion_sort(recs, b, e)
                ko, vo = oracle.sort(np.array(keys, dtype=np.uint64), np.arange(L), b, e)
                assert ko.tolist() == [r[0] for r in exp], (seq, b, e)
                assert vo.tolist() == [r[1] for r in exp], (seq, b, e)


# ---------------------------------------------------------------- library differential

def _np_stable(keys, vals, b, e):
    w = e - b
    sk = keys >> np.uint64(b) if b < 64 else np.zeros_like(keys)
    if w < 64:
        sk = sk & np.uint64((1 << w) - 1)
    order = np.argsort(sk, kind="stable")
    return keys[order], vals[order]


@pytest.mark.parametrize("bits", [32, 64])
@pytest.mark.parametrize("dist", ["uniform", "and3", "const"])
def test_numpy_stable_argsort_differential(bits, dist):
    for n, seed in ((1, 1), (31, 2), (1000, 3), (65537, 4)):
        k = oracle._u64(gen.keys(n, bits, dist, seed=seed))
        v = oracle._u64(gen.values(n, 64, "random", seed=seed))
        for b, e in [(0, bits), (0, 1), (7, 9), (8, 16), (1, bits - 1), (bits - 1, bits), (3, 3),
                     (0, 33 if bits == 64 else 32), (56, 64) if bits == 64 else (24, 32)]:
            ko, vo = oracle.sort(k, v, b, e)
            ek, ev = _np_stable(k, v, b, e)
            assert np.array_equal(ko, ek) and np.array_equal(vo, ev), (n, b, e)


def test_partition_pass_against_library():
    k = oracle._u64(gen.keys(5000, 64, "and2", seed=9))
    v = np.arange(5000, dtype=np.uint64)
    for lo, hi in ((56, 64), (0, 8), (3, 5), (60, 61)):
        ko, vo, offs = oracle.partition_pass(k, v, lo, hi)
        dig = (k >> np.uint64(lo)) & np.uint64((1 << (hi - lo)) - 1)
        order = np.argsort(dig, kind="stable")
        assert np.array_equal(ko, k[order]) and np.array_equal(vo, v[order])
        sd = np.sort(dig)
        assert offs.tolist() == np.searchsorted(sd, np.arange((1 << (hi - lo)) + 1), "left").tolist()


# ---------------------------------------------------------------- invariants

@pytest.mark.parametrize("bits,dist", [(32, "and4"), (64, "and3"), (32, "uniform")])
def test_invariants(bits, dist):
    n = 1 << 18
    k = oracle._u64(gen.keys(n, bits, dist, seed=11))
    v = np.arange(n, dtype=np.uint64)
    ko, vo = oracle.sort(k, v, 0, bits)
    # (1) non-decreasing
    assert np.all(ko[1:] >= ko[:-1])
    # (2) multiset equality via the full key histogram (np.unique = a sort-based count)
    u1, c1 = np.unique(k, return_counts=True)
    u2, c2 = np.unique(ko, return_counts=True)
    assert np.array_equal(u1, u2) and np.array_equal(c1, c2)
    # (3) stability: values (= input index) strictly increase inside every run of equal keys
    same = ko[1:] == ko[:-1]
    assert np.all(vo[1:][same] > vo[:-1][same])
    assert same.sum() > 0 or dist == "uniform"
    # certificate: key_out[i] == key_in[val_out[i]] (values form a permutation)
    assert np.array_equal(ko, k[vo.astype(np.int64)])


def test_begin_equals_end_is_identity_and_empty_ok():
    k = np.array([5, 3, 9], dtype=np.uint64)
    ko, vo = oracle.sort(k, np.arange(3), 4, 4)
    assert ko.tolist() == [5, 3, 9] and vo.tolist() == [0, 1, 2]
    ko, vo = oracle.sort(np.array([], dtype=np.uint64), np.array([], dtype=np.uint64), 0, 32)
    assert ko.size == 0


def test_torch_inputs_accepted():
    k = gen.keys(100, 32, "uniform")
    ko, _ = oracle.sort(k, None, 0, 32)
    assert np.all(ko[1:] >= ko[:-1])


# ---------------------------------------------------------------- bookkeeping (plan.py)

def test_merge_rule_worked_vector():
    """R3 with reading #5, ∂ = 4, ∂ˆ = 6, tot = [1,0,2,5,1,1,9,1]:
    1 + 2 = 3 < 4 merge {0,2}; 3 + 5 >= 4 closes; 5 alone, 5 + 1 >= 4 closes;
    1 + 1 = 2 < 4 merge {4,5}; 9 > ∂ˆ counts (and closes); 1 alone."""
    out = plan.classify_bucket([1, 0, 2, 5, 1, 1, 9, 1], False, 6, 4)
    assert out == [("local", [0, 2], 3), ("local", [3], 5), ("local", [4, 5], 2),
                   ("count", [6], 9), ("local", [7], 1)]
    assert plan.classify_bucket([1, 0, 2], True, 6, 4) == [("done", [0], 1), ("done", [2], 2)]


def test_size_classes():
    # [1,128] -> 0, (128,256] -> 1, (256,512] -> 2, and so on by powers of two
    assert [plan.size_class(s) for s in (1, 128, 129, 256, 257, 512, 513, 4096, 4097, 8192, 8193, 16384, 10**6)] == \
        [0, 0, 1, 1, 2, 2, 3, 5, 6, 6, 7, 7, 7]
    # another class table only relabels: boundaries are where the table says
    tab = (128, 256, 512, 1024, 2048, 4096, 4608, 8192)
    assert [plan.size_class(s, tab) for s in (4096, 4097, 4608, 4609, 8192)] == [5, 6, 6, 7, 7]


@pytest.mark.parametrize("dist", ["uniform", "and2", "and3", "and4", "const"])
@pytest.mark.parametrize("lt,mt,kpb", [(64, 40, 32), (300, 100, 128), (3, 2, 4)])
def test_msd_simulation_bounds_and_agreement(dist, lt, mt, kpb):
    """I1-I4 of P:817-836 hold and the MSD result equals the LSD oracle."""
    n = 4000
    k = oracle._u64(gen.keys(n, 32, dist, seed=5))
    v = np.arange(n, dtype=np.uint64)
    r = plan.simulate_msd(k, v, 0, 32, lt, mt, kpb)
    ko, vo = oracle.sort(k, v, 0, 32)
    assert np.array_equal(r.keys, ko) and np.array_equal(r.vals, vo)
    for p, (recs, tiles, nb) in enumerate(zip(r.recs_in_pass, r.tiles_in_pass, r.buckets_in_pass)):
        assert nb <= max(1, n // lt)                     # I1
        assert tiles <= n // kpb + n // lt + (p == 0)      # I4 (+1: the root bucket at pass 1)
    assert r.local_buckets <= min(2 * n // mt + n // lt, 256 * max(1, n // lt))  # I3
    for off, cnt, hi, c, p in r.local_entries:
        assert 1 <= cnt <= lt


def test_uniform_structure_prediction():
    """Uniform 2^20 u32 keys: after one pass the 256 buckets hold 4096 ± 64 (sigma) keys,
    so with ∂ˆ = 6144 there is exactly one counting pass and 256 local sorts."""
    n = 1 << 20
    k = oracle._u64(gen.keys(n, 32, "uniform"))
    r = plan.simulate_msd(k, None, 0, 32, 6144, 3000, 4096)
    assert r.counting_passes == 1 and r.local_buckets == 256 and r.merged_groups == 0
    assert plan.bytes_min(r, 4, 0) == 20 * n


def test_sort_typed_against_comparison_sort():
    """oracle.sort_typed (numpy) against a pure-Python stable comparison sort written from
    the documented order, on small inputs with the special values (±0, ±inf, NaN payloads,
    denormals, int min/max)."""
    import functools
    import struct
    rng = np.random.default_rng(5)
    ints = np.concatenate([rng.integers(-2**31, 2**31, 300), [-2**31, 2**31 - 1, 0, -1, 1, 0, -2**31]]).astype(np.int32)
    ek, ev = oracle.sort_typed(ints, np.arange(ints.size), "int")
    pairs = sorted(zip(ints.tolist(), range(ints.size)))  # (value, index) = stable numeric order
    assert ek.tolist() == [p[0] for p in pairs] and ev.tolist() == [p[1] for p in pairs]

    specials = [0.0, -0.0, np.inf, -np.inf, 1e-40, -1e-40, 1.5, -1.5, 0.0, -0.0]
    nans = [struct.unpack("<f", struct.pack("<I", b))[0] for b in (0x7FC00000, 0x7F800001, 0xFFC00000, 0xFF800001)]
    fl = np.concatenate([rng.standard_normal(200), specials, nans, specials]).astype(np.float32)
    bits = fl.view(np.uint32).tolist()

    def rank(i):  # documented total order as a tuple
        b = bits[i]
        neg, isnan = b >> 31, (b & 0x7F800000) == 0x7F800000 and (b & 0x7FFFFF) != 0
        if isnan:
            return (0, -b, i) if neg else (3, b, i)
        return (1 if neg else 2, float(fl[i]), i)

    def cmp(i, j):
        a, c = rank(i), rank(j)
        if a[0] != c[0]:
            return -1 if a[0] < c[0] else 1
        if a[1] != c[1]:
            return -1 if a[1] < c[1] else 1
        return -1 if i < j else (1 if i > j else 0)

    want = sorted(range(fl.size), key=functools.cmp_to_key(cmp))
    gk, gv = oracle.sort_typed(fl, np.arange(fl.size), "float")
    assert gv.tolist() == want
    assert gk.view(np.uint32).tolist() == [bits[i] for i in want]


# ---------------------------------------------------------------- std::stable_sort and the CPU baseline

@pytest.mark.parametrize("kbits,vbits", [(32, 0), (32, 32), (32, 64), (64, 0), (64, 32), (64, 64)])
@pytest.mark.parametrize("dist", ["uniform", "and3", "const"])
def test_oracle_equals_std_stable_sort_and_parallel_lsd(kbits, vbits, dist):
    """The library routine BJ north_star names: std::stable_sort of the (key, value)
    records by sk gives the oracle's bytes (a plausible oracle mistake -- a wrong digit
    order, an unstable scatter, a dropped narrow digit -- would differ).  The
    multi-threaded LSD (the timed CPU baseline) is byte-identical to the
    one-thread oracle for every thread count, including more threads than records."""
    n = 20011
    k = gen.keys(n, kbits, dist, seed=29)
    v = gen.values(n, vbits, "random", seed=29) if vbits else None
    kn = oracle._native(k)
    vn = oracle._native(v) if v is not None else None
    for b, e in ((0, kbits), (3, kbits - 5), (kbits - 1, kbits), (7, 7)):
        ek, ev = oracle.sort(kn, vn, b, e)
        sk, sv = oracle.cpu_stable_sort(kn, vn, b, e)
        assert np.array_equal(sk.astype(np.uint64), ek), (b, e)
        if v is not None:
            assert np.array_equal(sv.astype(np.uint64), ev), (b, e)
        for t in (1, 3, 8, 64):
            pk, pv = oracle.cpu_lsd_sort(kn, vn, b, e, threads=t)
            assert pk.dtype == kn.dtype
            assert np.array_equal(pk.astype(np.uint64), ek), (b, e, t)
            if v is not None:
                assert np.array_equal(pv.astype(np.uint64), ev), (b, e, t)
    # tiny inputs with more threads than records
    for n2 in (0, 1, 5):
        kk = kn[:n2].copy()
        pk, _ = oracle.cpu_lsd_sort(kk, None, 0, kbits, threads=16)
        assert np.array_equal(pk.astype(np.uint64), oracle.sort(kk, None, 0, kbits)[0])


def test_host_description():
    assert oracle.host_cores() >= 1
    assert isinstance(oracle.host_model(), str)


def test_leading_constant_digit_skip_rule():
    """Reading #22: a bucket still in the input whose digit is the same for all its records
    is not scattered (except in the last pass).  Closed forms: constant u32/u32 keys skip
    passes 1-3 and move once (4 x 4 B histogram reads + 16 B = 32 B/record); keys below
    2^24 skip pass 1 only; uniform keys never skip; a second constant digit after a real
    pass does not skip (the bucket moved)."""
    n = 50000
    lt, mt, kpb = 4096, 1024, 3072
    r = plan.simulate_msd(np.full(n, 0xA5A5A5A5, dtype=np.uint64), None, 0, 32, lt, mt, kpb)
    assert r.counting_passes == 4 and r.skipped_in_pass == [n, n, n, 0]
    assert plan.bytes_min(r, 4, 4) == 32 * n
    k = oracle._u64(gen.keys(n, 32, "uniform", seed=3)) & np.uint64(0x00FFFFFF)
    r = plan.simulate_msd(k, None, 0, 32, lt, mt, kpb)
    assert r.skipped_in_pass[0] == n and r.skipped_in_pass[1] == 0
    r = plan.simulate_msd(oracle._u64(gen.keys(n, 32, "uniform", seed=3)), None, 0, 32, lt, mt, kpb)
    assert r.counting_passes == 1 and r.skipped_in_pass == [0]
    assert plan.bytes_min(r, 4, 4) == 20 * n + 16 * n  # one pass (4 + 16 B) and the local sorts (16 B)
    # top digit varies, the second is constant: pass 2 moves (the buckets moved in pass 1)
    k = (oracle._u64(gen.keys(n, 32, "uniform", seed=4)) & np.uint64(0xFF00FFFF)) | np.uint64(0x00370000)
    r = plan.simulate_msd(k, None, 0, 32, 64, 16, 32)
    assert r.counting_passes >= 2 and r.skipped_in_pass[:2] == [0, 0]
    ks, _ = oracle.sort(k, None, 0, 32)
    assert np.array_equal(r.keys, ks)
