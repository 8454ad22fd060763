"""CPU oracle for the hybrid radix sort (arXiv 1611.01137) -- TEST INFRASTRUCTURE.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference
legs may import this package.  The product library (paper_1611_01137_b200) never
imports it, and the two share no code: the only common module is gen/ (seeded
input generators, none of the method's arithmetic).

Contents
  oracle.c (built to liboracle.so, loaded with ctypes):
      histogram       -- digit histogram, P:293-296 / P:503-505
      partition_pass  -- one stable counting-sort pass, P:293-301 / P:503-509
      sort            -- LSD radix sort, 8-bit digits, P:304-311 (the definition of
                         the unique stable sort by bits [begin, end))
  plan.py (pure Python):
      classify_bucket -- rules R1-R3 and tiny-bucket merging, P:552-561, P:805-811
      simulate_msd    -- the MSD hybrid recursion step by step (Fig 1),
                         giving the pass / bucket / local-sort structure

Pinning (none of these re-run the oracle's own formula): tests/test_oracle.py
checks the paper's worked example (Table 2, tests/golden/table2.txt),
brute force against insertion sort on every short sequence over a 4-letter
alphabet, numpy's stable argsort (a library routine), and the invariants
non-decreasing / multiset equality / stability.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_CPU_SRC = os.path.join(_HERE, "cpu_baseline.cc")
_CPU_LIB = os.path.join(_HERE, "libcpu_baseline.so")
_lib = None
_cpu = None


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (plain C, -O2, single thread) and cpu_baseline.cc with g++
    (the multi-threaded LSD baseline and the std::stable_sort cross-check)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        subprocess.check_call(["gcc", "-O2", "-std=c99", "-shared", "-fPIC", "-o", _LIB, _SRC])
    if force or not os.path.exists(_CPU_LIB) or os.path.getmtime(_CPU_LIB) < os.path.getmtime(_CPU_SRC):
        subprocess.check_call(["g++", "-O3", "-std=c++17", "-pthread", "-shared", "-fPIC", "-o", _CPU_LIB,
                               _CPU_SRC])
    return _LIB


def _load_cpu():
    global _cpu
    if _cpu is None:
        build()
        lib = ctypes.CDLL(_CPU_LIB)
        P, U, I = ctypes.c_void_p, ctypes.c_uint64, ctypes.c_int
        lib.cpu_lsd_sort.argtypes = [P, P, U, I, I, I, I, P, P, I]
        lib.cpu_stable_sort.argtypes = [P, P, U, I, I, I, I, P, P]
        lib.cpu_lsd_sort.restype = I
        lib.cpu_stable_sort.restype = I
        _cpu = lib
    return _cpu


def host_cores() -> int:
    """Cores this process may run on (sched_getaffinity), the baseline's thread count."""
    try:
        return len(os.sched_getaffinity(0))
    except AttributeError:  # pragma: no cover
        return os.cpu_count() or 1


def host_model() -> str:
    """CPU model name (lscpu / /proc/cpuinfo), for the cpu_baseline record."""
    try:
        for line in open("/proc/cpuinfo", encoding="utf-8"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip()
    except OSError:  # pragma: no cover
        pass
    return "unknown"


def _native(a):
    """A numpy uint32/uint64 view of a numpy array or torch CPU tensor (no widening)."""
    if hasattr(a, "numpy"):
        a = a.cpu()
        import torch
        if a.dtype == torch.uint32:
            return a.view(torch.int32).numpy().view(np.uint32)
        if a.dtype == torch.uint64:
            return a.view(torch.int64).numpy().view(np.uint64)
        a = a.numpy()
    a = np.ascontiguousarray(a)
    if a.dtype not in (np.uint32, np.uint64):
        raise TypeError(a.dtype)
    return a


def cpu_lsd_sort(keys, vals=None, begin_bit: int = 0, end_bit: int | None = None, threads: int | None = None):
    """Multi-threaded stable LSD radix sort (the timed CPU baseline) on the
    native widths; byte-identical to sort() for any thread count."""
    k = _native(keys)
    v = _native(vals) if vals is not None else None
    if end_bit is None:
        end_bit = 8 * k.itemsize
    ko = np.empty_like(k)
    vo = np.empty_like(v) if v is not None else None
    rc = _load_cpu().cpu_lsd_sort(_ptr(k), _ptr(v), k.size, k.itemsize, 0 if v is None else v.itemsize, begin_bit,
                                  end_bit, _ptr(ko), _ptr(vo), threads or host_cores())
    if rc:
        raise ValueError(f"cpu_lsd_sort rc={rc}")
    return ko, vo


def cpu_stable_sort(keys, vals=None, begin_bit: int = 0, end_bit: int | None = None):
    """std::stable_sort of the (key, value) records by key bits [begin, end), one thread."""
    k = _native(keys)
    v = _native(vals) if vals is not None else None
    if end_bit is None:
        end_bit = 8 * k.itemsize
    ko = np.empty_like(k)
    vo = np.empty_like(v) if v is not None else None
    rc = _load_cpu().cpu_stable_sort(_ptr(k), _ptr(v), k.size, k.itemsize, 0 if v is None else v.itemsize,
                                     begin_bit, end_bit, _ptr(ko), _ptr(vo))
    if rc:
        raise ValueError(f"cpu_stable_sort rc={rc}")
    return ko, vo


def _load():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB)
        P = ctypes.c_void_p
        U = ctypes.c_uint64
        I = ctypes.c_int
        lib.oracle_digit_histogram.argtypes = [P, U, I, I, P]
        lib.oracle_partition_pass.argtypes = [P, P, U, I, I, P, P, P]
        lib.oracle_lsd_sort.argtypes = [P, P, U, I, I, P, P]
        for f in (lib.oracle_digit_histogram, lib.oracle_partition_pass, lib.oracle_lsd_sort):
            f.restype = I
        _lib = lib
    return _lib


def _u64(a) -> np.ndarray:
    """Widen any unsigned integer array (numpy or torch CPU tensor) to contiguous uint64."""
    if hasattr(a, "numpy"):  # torch tensor
        a = a.cpu()
        if str(a.dtype) == "torch.uint32":
            a = a.view(dtype=__import__("torch").int32).numpy().view(np.uint32)
        elif str(a.dtype) == "torch.uint64":
            a = a.view(dtype=__import__("torch").int64).numpy().view(np.uint64)
        else:
            a = a.numpy()
    a = np.asarray(a)
    if a.dtype.kind not in "ui":
        raise TypeError(a.dtype)
    return np.ascontiguousarray(a.astype(np.uint64, copy=False))


def _ptr(a: np.ndarray):
    return a.ctypes.data_as(ctypes.c_void_p) if a is not None else None


def histogram(keys, lo: int, hi: int) -> np.ndarray:
    k = _u64(keys)
    h = np.zeros(1 << (hi - lo), dtype=np.uint64)
    rc = _load().oracle_digit_histogram(_ptr(k), k.size, lo, hi, _ptr(h))
    if rc:
        raise ValueError(f"oracle_digit_histogram rc={rc}")
    return h


def partition_pass(keys, vals, lo: int, hi: int):
    """One stable counting pass on digit bits [lo, hi): (keys_out, vals_out, offsets[r+1])."""
    k = _u64(keys)
    v = _u64(vals) if vals is not None else None
    ko = np.empty_like(k)
    vo = np.empty_like(v) if v is not None else None
    offs = np.zeros((1 << (hi - lo)) + 1, dtype=np.uint64)
    rc = _load().oracle_partition_pass(_ptr(k), _ptr(v), k.size, lo, hi, _ptr(ko), _ptr(vo), _ptr(offs))
    if rc:
        raise ValueError(f"oracle_partition_pass rc={rc}")
    return ko, vo, offs


def sort(keys, vals=None, begin_bit: int = 0, end_bit: int | None = None, key_bits: int | None = None):
    """The stable sort by bits [begin_bit, end_bit) -> (keys_out, vals_out) as uint64 arrays."""
    k = _u64(keys)
    if end_bit is None:
        end_bit = key_bits if key_bits is not None else 64
    v = _u64(vals) if vals is not None else None
    ko = np.empty_like(k)
    vo = np.empty_like(v) if v is not None else None
    rc = _load().oracle_lsd_sort(_ptr(k), _ptr(v), k.size, begin_bit, end_bit, _ptr(ko), _ptr(vo))
    if rc:
        raise ValueError(f"oracle_lsd_sort rc={rc}")
    return ko, vo


from .plan import classify_bucket, simulate_msd, size_class  # noqa: E402,F401


def sort_typed(keys, vals, kind: str):
    """Stable sort of signed ('int') or IEEE-754 ('float') keys by value, the order
    include/hrs.h documents for hrs_sort_typed (the paper's P:907-918 bijections define
    the GPU side; this is the plain definition, independent of them):
      int:   two's-complement numeric order;
      float: -NaN (larger bit pattern first) < -inf < ... < -0.0 < +0.0 < ... < +inf <
             +NaN (smaller bit pattern first); equal keys keep input order.
    keys: numpy int32/int64/float32/float64 array; returns (keys_out, vals_out)."""
    k = np.asarray(keys)
    v = None if vals is None else np.asarray(vals)
    idx = np.arange(k.size)
    if kind == "int":
        order = np.argsort(k, kind="stable")
    elif kind == "float":
        ub = np.uint32 if k.dtype == np.float32 else np.uint64
        bits = k.view(ub).astype(np.uint64)
        sign = (bits >> np.uint64(8 * k.itemsize - 1)).astype(np.int64)
        nan = np.isnan(k)
        neg_nan, pos_nan, num = idx[nan & (sign == 1)], idx[nan & (sign == 0)], idx[~nan]
        order = np.concatenate([
            neg_nan[np.lexsort((neg_nan, ~bits[neg_nan]))],       # further from zero first
            num[np.lexsort((num, 1 - sign[num], k[num]))],       # value, then -0.0 before +0.0
            pos_nan[np.lexsort((pos_nan, bits[pos_nan]))]]).astype(np.int64)
    else:
        raise ValueError(kind)
    return k[order], (None if v is None else v[order])
