"""ctypes binding of libhrs.so (include/hrs.h).  Argument marshalling only.

There is deliberately no fallback: if the shared library is missing the import
fails loudly (build it with ``python paper_1611_01137_b200/build.py``).
"""
from __future__ import annotations

import ctypes
import os

HERE = os.path.dirname(os.path.abspath(__file__))
# HRS_LIB overrides the library path (used only by the kernel-variant experiments in micro/)
LIB_PATH = os.environ.get("HRS_LIB") or os.path.join(HERE, "libhrs.so")

HRS_MAX_PASSES = 8
HRS_NUM_CLASSES = 8
HRS_MAX_ITEMS = 0xFFFFFFFF

STATUS_NAMES = {
    0: "HRS_SUCCESS",
    1: "HRS_ERROR_INVALID_VALUE",
    2: "HRS_ERROR_INVALID_BITS",
    3: "HRS_ERROR_ALIASING",
    4: "HRS_ERROR_TEMP_TOO_SMALL",
    5: "HRS_ERROR_TOO_LARGE",
    6: "HRS_ERROR_NO_DEVICE",
    7: "HRS_ERROR_CUDA",
}


class HrsError(RuntimeError):
    def __init__(self, status: int, message: str):
        super().__init__(f"{STATUS_NAMES.get(status, status)}: {message}")
        self.status = status


class Tuning(ctypes.Structure):
    """hrs_tuning: 0 in a field selects the default."""
    _fields_ = [
        ("local_threshold", ctypes.c_uint32),
        ("merge_threshold", ctypes.c_uint32),
        ("keys_per_tile", ctypes.c_uint32),
        ("local_classes", ctypes.c_uint32),
        ("flags", ctypes.c_uint32),
    ]


HRS_FLAG_FORCE_REDO = 1


class Stats(ctypes.Structure):
    _fields_ = [
        ("n", ctypes.c_uint64),
        ("key_bytes", ctypes.c_uint32),
        ("value_bytes", ctypes.c_uint32),
        ("counting_passes", ctypes.c_uint32),
        ("overflow", ctypes.c_uint32),
        ("recs_in_pass", ctypes.c_uint64 * HRS_MAX_PASSES),
        ("tiles_in_pass", ctypes.c_uint64 * HRS_MAX_PASSES),
        ("buckets_in_pass", ctypes.c_uint64 * HRS_MAX_PASSES),
        ("local_buckets", ctypes.c_uint64),
        ("local_recs", ctypes.c_uint64),
        ("merged_groups", ctypes.c_uint64),
        ("local_in_class", ctypes.c_uint64 * HRS_NUM_CLASSES),
        ("bytes_min", ctypes.c_uint64),
        ("redo_blocks", ctypes.c_uint64),
        ("skipped_recs_in_pass", ctypes.c_uint64 * HRS_MAX_PASSES),
    ]

    def to_dict(self) -> dict:
        p = self.counting_passes
        return {
            "n": self.n,
            "key_bytes": self.key_bytes,
            "value_bytes": self.value_bytes,
            "counting_passes": p,
            "overflow": self.overflow,
            "recs_in_pass": list(self.recs_in_pass)[:p],
            "tiles_in_pass": list(self.tiles_in_pass)[:p],
            "buckets_in_pass": list(self.buckets_in_pass)[:p],
            "local_buckets": self.local_buckets,
            "local_recs": self.local_recs,
            "merged_groups": self.merged_groups,
            "local_in_class": list(self.local_in_class),
            "bytes_min": self.bytes_min,
            "redo_blocks": self.redo_blocks,
            "skipped_recs_in_pass": list(self.skipped_recs_in_pass)[:p],
        }


class ProfileRecord(ctypes.Structure):
    _fields_ = [("kind", ctypes.c_int), ("pass_", ctypes.c_int), ("ms", ctypes.c_float)]


PROFILE_KINDS = {0: "init", 1: "hist", 2: "scatter", 3: "local", 4: "copy", 5: "classify"}

# name -> (restype, argtypes); mirrors include/hrs.h exactly (tests check the header)
_P = ctypes.c_void_p
_U64 = ctypes.c_uint64
_I = ctypes.c_int
_SZP = ctypes.POINTER(ctypes.c_size_t)
_ST = ctypes.c_int
SIGNATURES = {
    "hrs_sort_keys_u32": (_ST, [_P, _SZP, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_keys_u64": (_ST, [_P, _SZP, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_pairs_u32_u32": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_pairs_u32_u64": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_pairs_u64_u32": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_pairs_u64_u64": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _P]),
    "hrs_sort_ex": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _I, _I, ctypes.POINTER(Tuning), _P]),
    "hrs_sort_typed": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _I, _P]),
    "hrs_sort_records": (_ST, [_P, _SZP, _P, _P, _U64, _I, _I, _I, _I, _I, _I, _P]),
    "hrs_sort_grouped": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _I, _I, _P, ctypes.POINTER(Tuning), _P]),
    "hrs_get_stats": (_ST, [_P, ctypes.POINTER(Stats), _P]),
    "hrs_max_local_threshold": (ctypes.c_uint32, [_I, _I]),
    "hrs_max_keys_per_tile": (ctypes.c_uint32, [_I, _I]),
    "hrs_default_tuning": (_ST, [_I, _I, ctypes.POINTER(Tuning)]),
    "hrs_class_capacity": (ctypes.c_uint32, [_I]),
    "hrs_digit_histogram": (_ST, [_P, _SZP, _P, _U64, _I, _I, _I, _P, _P]),
    "hrs_partition_pass": (_ST, [_P, _SZP, _P, _P, _P, _P, _U64, _I, _I, _I, _I, _P, _P]),
    "hrs_copy_pieces": (_ST, [_P, _P, _I, _P, _U64, _P]),
    "hrs_partition_pass_to": (_ST, [_P, _SZP, _P, _P, _U64, _I, _I, _I, _I, _P, _I, _P, _P, _P]),
    "hrs_profile_enable": (None, [_I]),
    "hrs_profile_collect": (_I, [ctypes.POINTER(ProfileRecord), _I]),
    "hrs_launch_count": (ctypes.c_uint64, []),
    "hrs_status_string": (ctypes.c_char_p, [_ST]),
    "hrs_last_cuda_error": (_I, []),
    "hrs_version": (_I, []),
}


def load(path: str = LIB_PATH) -> ctypes.CDLL:
    if not os.path.exists(path):
        raise ImportError(
            f"{path} is missing: the CUDA library is required (there is no CPU fallback). "
            "Build it with `python paper_1611_01137_b200/build.py`.")
    lib = ctypes.CDLL(path)
    for name, (res, args) in SIGNATURES.items():
        f = getattr(lib, name)
        f.restype = res
        f.argtypes = args
    return lib


lib = load()


def check(status: int, what: str) -> None:
    if status != 0:
        msg = lib.hrs_status_string(status).decode()
        if status == 7:
            msg += f" (cudaError {lib.hrs_last_cuda_error()})"
        raise HrsError(status, f"{what}: {msg}")
