"""Seeded synthetic workload generators shared by the oracle tests and the CUDA path.

This module holds NONE of the sorting method's arithmetic: it only produces input
keys and values.  It is the single piece of code both sides may use (the oracle
and the CUDA library share nothing else).

Workload shape (§6): keys are uniform, or skewed by AND-ing
m uniform draws (Thearling & Smith), which leaves every bit set with probability
2^-m and gives an entropy of kb * H(2^-m) bits per key (P:1036-1039 prints
25.96 / 17.39 / 10.79 bits for 32-bit keys and m = 2 / 3 / 4).  "Constant" keys
(0-bit entropy) are all zero.

The uniform source is the counter-based splitmix64 of SURVEY.md §8(d):

    splitmix64(x): z = x + 0x9E3779B97F4A7C15
                   z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9
                   z = (z ^ (z >> 27)) * 0x94D049BB133111EB
                   return z ^ (z >> 31)
    stream_j = splitmix64(seed ^ (0xD1B54A32D192ED03 * (j + 1)))     j = 0..m-1
    u_j(i)   = splitmix64(stream_j + i)                              i = global index
    key(i)   = u_0(i) & ... & u_{m-1}(i)   truncated to kb bits
    value(i) = splitmix64((seed ^ 0x5A5A5A5A5A5A5A5A) + i) truncated  (or i itself)

All arithmetic is mod 2^64.  It is written with torch int64 tensor ops (wrapping
two's-complement multiply, masked logical shifts) so the *same code* runs on the
CPU and on a CUDA device and yields identical bytes; any record can be regenerated
from its global index, which the O(n) certificate checks rely on.
"""
from __future__ import annotations

import math

import torch

M64 = (1 << 64) - 1

SEEDS = (0x1611011370000001, 0x1611011370000002, 0x1611011370000003)

_GOLDEN = 0x9E3779B97F4A7C15
_MIX1 = 0xBF58476D1CE4E5B9
_MIX2 = 0x94D049BB133111EB
_STREAM = 0xD1B54A32D192ED03
_VALSALT = 0x5A5A5A5A5A5A5A5A

DISTS = ("uniform", "and2", "and3", "and4", "const")


def _s64(x: int) -> int:
    """Reinterpret an unsigned 64-bit integer as signed (for torch int64 constants)."""
    x &= M64
    return x - (1 << 64) if x >> 63 else x


def splitmix64_int(x: int) -> int:
    """Pure-Python splitmix64 on one integer (the reference for the tensor form)."""
    z = (x + _GOLDEN) & M64
    z = ((z ^ (z >> 30)) * _MIX1) & M64
    z = ((z ^ (z >> 27)) * _MIX2) & M64
    return z ^ (z >> 31)


def _srl(z: torch.Tensor, s: int) -> torch.Tensor:
    """Logical right shift of an int64 tensor holding uint64 bit patterns."""
    return (z >> s) & ((1 << (64 - s)) - 1)


def splitmix64(x: torch.Tensor) -> torch.Tensor:
    """splitmix64 on an int64 tensor of uint64 bit patterns (wrapping arithmetic)."""
    z = x + _s64(_GOLDEN)
    z = (z ^ _srl(z, 30)) * _s64(_MIX1)
    z = (z ^ _srl(z, 27)) * _s64(_MIX2)
    return z ^ _srl(z, 31)


def stream_seed(seed: int, j: int) -> int:
    return splitmix64_int((seed ^ ((_STREAM * (j + 1)) & M64)) & M64)


def and_count(dist: str) -> int:
    """Number m of uniform draws AND-ed together (0 = constant keys)."""
    if dist == "uniform":
        return 1
    if dist == "const":
        return 0
    if dist.startswith("and"):
        m = int(dist[3:])
        if m < 1:
            raise ValueError(dist)
        return m
    raise ValueError(f"unknown distribution {dist!r}")


def entropy_bits(key_bits: int, m: int) -> float:
    """Closed-form entropy per key of AND-m keys: kb * H(2^-m)."""
    if m == 0:
        return 0.0
    p = 2.0 ** -m
    if p == 1.0:
        return 0.0
    h = -(p * math.log2(p) + (1 - p) * math.log2(1 - p))
    return key_bits * h


def _as_unsigned(x64: torch.Tensor, bits: int) -> torch.Tensor:
    if bits == 64:
        return x64.view(torch.uint64)
    if bits == 32:
        return x64.to(torch.int32).view(torch.uint32)
    raise ValueError(bits)


def _chunks(start: int, n: int, chunk: int):
    i = 0
    while i < n:
        c = min(chunk, n - i)
        yield start + i, i, c
        i += c


def keys(n: int, key_bits: int = 32, dist: str = "uniform", seed: int = SEEDS[0],
         start: int = 0, device="cpu", chunk: int = 1 << 24) -> torch.Tensor:
    """Keys for global indices [start, start + n) as a uint32/uint64 tensor."""
    m = and_count(dist)
    out = torch.empty(n, dtype=torch.int64, device=device)
    if m == 0:
        out.zero_()
        return _as_unsigned(out, key_bits)
    streams = [_s64(stream_seed(seed, j)) for j in range(m)]
    for g0, o0, c in _chunks(start, n, chunk):
        idx = torch.arange(g0, g0 + c, dtype=torch.int64, device=device)
        acc = splitmix64(idx + streams[0])
        for j in range(1, m):
            acc &= splitmix64(idx + streams[j])
        out[o0:o0 + c] = acc
    return _as_unsigned(out, key_bits)


def values(n: int, value_bits: int = 32, kind: str = "random", seed: int = SEEDS[0],
           start: int = 0, device="cpu", chunk: int = 1 << 24) -> torch.Tensor:
    """Values for global indices [start, start + n): 'index' (= i) or 'random'."""
    out = torch.empty(n, dtype=torch.int64, device=device)
    if kind == "index":
        torch.arange(start, start + n, dtype=torch.int64, device=device, out=out)
        return _as_unsigned(out, value_bits)
    if kind != "random":
        raise ValueError(kind)
    base = _s64(seed ^ _VALSALT)
    for g0, o0, c in _chunks(start, n, chunk):
        idx = torch.arange(g0, g0 + c, dtype=torch.int64, device=device)
        out[o0:o0 + c] = splitmix64(idx + base)
    return _as_unsigned(out, value_bits)


def key_ref(i: int, key_bits: int = 32, dist: str = "uniform", seed: int = SEEDS[0]) -> int:
    """Pure-Python key of global index i (for spot checks at any size)."""
    m = and_count(dist)
    if m == 0:
        return 0
    acc = M64
    for j in range(m):
        acc &= splitmix64_int((stream_seed(seed, j) + i) & M64)
    return acc & ((1 << key_bits) - 1)


def value_ref(i: int, value_bits: int = 32, kind: str = "random", seed: int = SEEDS[0]) -> int:
    if kind == "index":
        return i & ((1 << value_bits) - 1)
    return splitmix64_int(((seed ^ _VALSALT) + i) & M64) & ((1 << value_bits) - 1)
