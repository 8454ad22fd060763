"""Generator pins (CPU): splitmix64 known answer, closed-form entropy, per-bit rates."""
import math

import numpy as np
import pytest
import torch

import gen


def test_splitmix64_known_answer():
    # splitmix64 (Steele, Lea & Flood) seeded with 0: first output is 0xE220A8397B1DCDAF,
    # second 0x6E789E6AA1B965F4 (state advanced by the golden gamma each call).
    assert gen.splitmix64_int(0) == 0xE220A8397B1DCDAF
    assert gen.splitmix64_int(0x9E3779B97F4A7C15) == 0x6E789E6AA1B965F4


def test_tensor_form_matches_integer_form():
    xs = [0, 1, 2, 0x7FFFFFFFFFFFFFFF, 0x8000000000000000, 0xFFFFFFFFFFFFFFFF, 0x123456789ABCDEF0]
    t = torch.tensor([gen._s64(x) for x in xs], dtype=torch.int64)
    got = [int(v) & gen.M64 for v in gen.splitmix64(t).tolist()]
    assert got == [gen.splitmix64_int(x) for x in xs]


@pytest.mark.parametrize("dist", ["uniform", "and2", "and3", "const"])
@pytest.mark.parametrize("bits", [32, 64])
def test_keys_match_reference_per_index(dist, bits):
    n, start = 257, 1 << 33
    k = gen.keys(n, bits, dist, start=start)
    kk = k.view(torch.int32 if bits == 32 else torch.int64).numpy().view(np.uint32 if bits == 32 else np.uint64)
    for i in (0, 1, 100, 256):
        assert int(kk[i]) == gen.key_ref(start + i, bits, dist)


def test_values_reference():
    v = gen.values(64, 64, "random", start=5)
    vv = v.view(torch.int64).numpy().view(np.uint64)
    assert int(vv[3]) == gen.value_ref(8, 64, "random")
    vi = gen.values(10, 32, "index", start=7)
    assert vi.view(torch.int32).tolist() == list(range(7, 17))


def test_chunking_is_invisible():
    a = gen.keys(1000, 64, "and2", chunk=1 << 20)
    b = gen.keys(1000, 64, "and2", chunk=97)
    assert torch.equal(a.view(torch.int64), b.view(torch.int64))


def test_entropy_closed_form_matches_paper():
    # AND-ing once, twice, three times -> 25.96, 17.39, 10.79 bits (32-bit keys)
    assert round(gen.entropy_bits(32, 2), 2) == 25.96
    assert round(gen.entropy_bits(32, 3), 2) == 17.39
    assert round(gen.entropy_bits(32, 4), 2) == 10.79
    # 64-bit axis of Figs 7/12: 51.92 / 34.79 / 21.59
    assert round(gen.entropy_bits(64, 2), 2) == 51.92
    assert round(gen.entropy_bits(64, 3), 2) == 34.79
    assert round(gen.entropy_bits(64, 4), 2) == 21.59
    assert gen.entropy_bits(32, 1) == 32.0


@pytest.mark.parametrize("m", [1, 2, 3, 4])
def test_bit_rate_is_two_to_minus_m(m):
    n = 1 << 16
    k = gen.keys(n, 64, "uniform" if m == 1 else f"and{m}").view(torch.int64)
    p = 2.0 ** -m
    sigma = math.sqrt(n * p * (1 - p))
    for b in (0, 7, 31, 32, 63):
        cnt = int(((k >> b) & 1).sum())
        assert abs(cnt - n * p) < 4.5 * sigma, (m, b, cnt)
