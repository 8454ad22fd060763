"""B200-native (sm_100a) stable hybrid MSD radix sort -- Python binding.

Implements the hot path of Stehle & Jacobsen, "A Memory Bandwidth-Efficient Hybrid
Radix Sort on GPUs" (arXiv 1611.01137): MSD counting-sort passes on 8-bit digits
(histogram -> exclusive prefix sum -> shared-memory staged scatter), recursion on
buckets above the local-sort threshold, tiny-bucket merging and an on-chip local
sort.  Every step runs in the CUDA kernels of libhrs.so (include/hrs.h); this
module only allocates with torch and marshals arguments through ctypes.
"""
from __future__ import annotations

import ctypes

import torch

from ._lib import HRS_MAX_ITEMS, HrsError, Stats, Tuning, check, lib  # noqa: F401

__all__ = ["sort", "sort_grouped", "sort_records", "temp_bytes", "get_stats", "digit_histogram", "partition_pass", "HrsError", "Tuning",
           "default_tuning", "max_local_threshold", "max_keys_per_tile", "class_capacities", "lib"]

_KEY_DTYPES = {torch.uint32: 4, torch.uint64: 8}
# signed / floating-point keys: (key bytes, hrs_key_kind) -- hrs_sort_typed
_TYPED_KEYS = {torch.int32: (4, 1), torch.int64: (8, 1), torch.float32: (4, 2), torch.float64: (8, 2)}


def _nbytes(t: torch.Tensor | None, what: str) -> int:
    if t is None:
        return 0
    if t.dtype not in _KEY_DTYPES:
        raise TypeError(f"{what} must be torch.uint32 or torch.uint64, got {t.dtype}")
    return _KEY_DTYPES[t.dtype]


def _check_tensor(t: torch.Tensor, what: str) -> None:
    if not t.is_cuda:
        raise ValueError(f"{what} must be a CUDA tensor (there is no CPU path)")
    if not t.is_contiguous():
        raise ValueError(f"{what} must be contiguous")
    if t.dim() != 1:
        raise ValueError(f"{what} must be 1-D")


def _ptr(t: torch.Tensor | None):
    return ctypes.c_void_p(t.data_ptr()) if t is not None and t.numel() > 0 else ctypes.c_void_p(0)


def _stream(stream) -> ctypes.c_void_p:
    if stream is None:
        stream = torch.cuda.current_stream()
    return ctypes.c_void_p(stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream))


def _on_stream(stream, *tensors) -> None:
    """Tensors the binding allocated (on torch's current stream) but the library uses on
    `stream`: tell the caching allocator, so a block freed on return is not handed to a
    new allocation while the sort is still running on `stream`."""
    if stream is None or not isinstance(stream, torch.cuda.Stream):
        return
    if stream == torch.cuda.current_stream(stream.device):
        return
    for t in tensors:
        if t is not None:
            t.record_stream(stream)


def _out(t: torch.Tensor | None, like: torch.Tensor, what: str) -> torch.Tensor:
    """An output buffer: allocated like `like`, or the caller's, checked for length, dtype
    and device (the library writes n elements through the raw pointer)."""
    if t is None:
        return torch.empty_like(like)
    _check_tensor(t, what)
    if t.dtype != like.dtype or t.numel() != like.numel() or t.device != like.device:
        raise ValueError(f"{what} must be a {like.dtype} tensor of {like.numel()} elements on {like.device}, "
                         f"got {t.dtype} x {t.numel()} on {t.device}")
    return t


def _tuning(tuning) -> ctypes.POINTER(Tuning) | None:
    if tuning is None:
        return None
    if isinstance(tuning, dict):
        tuning = Tuning(**tuning)
    return ctypes.pointer(tuning)


def temp_bytes(n: int, key_bytes: int, value_bytes: int = 0, begin_bit: int = 0, end_bit: int | None = None,
               tuning=None) -> int:
    """Required temp size for a sort (the library's two-phase temp protocol)."""
    if end_bit is None:
        end_bit = 8 * key_bytes
    sz = ctypes.c_size_t(0)
    check(lib.hrs_sort_ex(None, ctypes.byref(sz), None, None, None, None, n, key_bytes, value_bytes, begin_bit,
                          end_bit, _tuning(tuning), None), "hrs_sort_ex(size query)")
    return sz.value


def alloc_temp(nbytes: int, device) -> torch.Tensor:
    return torch.empty(max(nbytes, 256), dtype=torch.uint8, device=device)


def sort(keys: torch.Tensor, values: torch.Tensor | None = None, begin_bit: int = 0, end_bit: int | None = None,
         *, tuning=None, keys_out: torch.Tensor | None = None, values_out: torch.Tensor | None = None,
         temp: torch.Tensor | None = None, stream=None, first_digit_hist: torch.Tensor | None = None):
    """Stable sort of `keys` (and `values`) by key bits [begin_bit, end_bit).

    Returns (keys_out, values_out); values_out is None for keys-only sorts.
    Enqueued on `stream` (default: torch's current stream); nothing synchronises.
    """
    _check_tensor(keys, "keys")
    if keys.dtype in _TYPED_KEYS:
        if first_digit_hist is not None:
            raise TypeError("grouped sorts take unsigned keys")
        return sort_typed(keys, values, keys_out=keys_out, values_out=values_out, temp=temp, stream=stream,
                          begin_bit=begin_bit, end_bit=end_bit, tuning=tuning)
    kb = _nbytes(keys, "keys")
    vb = 0
    if values is not None:
        _check_tensor(values, "values")
        vb = _nbytes(values, "values")
        if values.numel() != keys.numel():
            raise ValueError("keys and values differ in length")
        if values.device != keys.device:
            raise ValueError("keys and values are on different devices")
    n = keys.numel()
    if end_bit is None:
        end_bit = 8 * kb
    keys_out = _out(keys_out, keys, "keys_out")
    if values is not None:
        values_out = _out(values_out, values, "values_out")
    tb = temp_bytes(n, kb, vb, begin_bit, end_bit, tuning)
    if temp is None or temp.numel() < tb:
        temp = alloc_temp(tb, keys.device)
    _on_stream(stream, temp, keys_out, values_out)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(keys.device):
        if first_digit_hist is None:
            check(lib.hrs_sort_ex(_ptr(temp), ctypes.byref(sz), _ptr(keys), _ptr(keys_out), _ptr(values),
                                  _ptr(values_out), n, kb, vb, begin_bit, end_bit, _tuning(tuning),
                                  _stream(stream)), "hrs_sort_ex")
        else:
            check(lib.hrs_sort_grouped(_ptr(temp), ctypes.byref(sz), _ptr(keys), _ptr(keys_out), _ptr(values),
                                       _ptr(values_out), n, kb, vb, begin_bit, end_bit, _ptr(first_digit_hist),
                                       _tuning(tuning), _stream(stream)), "hrs_sort_grouped")
    return keys_out, (values_out if values is not None else None)


def sort_grouped(keys: torch.Tensor, values: torch.Tensor | None, first_digit_hist, begin_bit: int = 0,
                 end_bit: int | None = None, **kw):
    """hrs_sort_grouped: the stable sort of an input already grouped by its first digit
    (bits [max(begin, end - 8), end)) in ascending order, with that digit's counts
    `first_digit_hist` (a sequence or a tensor of 2^width counts); skips the first pass."""
    if keys.dtype in _TYPED_KEYS:
        raise TypeError("sort_grouped takes unsigned keys")
    if end_bit is None:
        end_bit = 8 * _nbytes(keys, "keys")
    width = min(8, end_bit - begin_bit)
    h = first_digit_hist
    if not isinstance(h, torch.Tensor) or h.dtype != torch.uint64 or not h.is_cuda:
        h = torch.as_tensor([int(x) for x in (h.tolist() if isinstance(h, torch.Tensor) else h)],
                            dtype=torch.int64).view(torch.uint64).to(keys.device)
    if end_bit > begin_bit and h.numel() != (1 << width):
        raise ValueError(f"first_digit_hist needs {1 << width} counts")
    stream = kw.get("stream")
    _on_stream(stream, h)
    return sort(keys, values, begin_bit, end_bit, first_digit_hist=h, **kw)


def typed_temp_bytes(n: int, key_bytes: int, value_bytes: int, kind: int) -> int:
    sz = ctypes.c_size_t(0)
    check(lib.hrs_sort_typed(None, ctypes.byref(sz), None, None, None, None, n, key_bytes, value_bytes, kind, None),
          "hrs_sort_typed")
    return sz.value


def sort_typed(keys: torch.Tensor, values: torch.Tensor | None = None, *, keys_out=None, values_out=None, temp=None,
               stream=None, begin_bit: int = 0, end_bit: int | None = None, tuning=None):
    """Stable sort of int32/int64 (two's complement) or float32/float64 (IEEE-754 total
    order, -0.0 < +0.0, NaNs at the ends by sign) keys by their whole value, with
    uint32/uint64 values moved along."""
    _check_tensor(keys, "keys")
    if keys.dtype not in _TYPED_KEYS:
        raise TypeError(f"keys must be int32/int64/float32/float64 here, got {keys.dtype}")
    kb, kind = _TYPED_KEYS[keys.dtype]
    if begin_bit != 0 or (end_bit is not None and end_bit != 8 * kb) or tuning is not None:
        raise ValueError("signed/float keys sort by the whole key (no bit range, no tuning)")
    vb = 0
    if values is not None:
        _check_tensor(values, "values")
        vb = _nbytes(values, "values")
        if values.numel() != keys.numel():
            raise ValueError("keys and values differ in length")
    n = keys.numel()
    keys_out = _out(keys_out, keys, "keys_out")
    if values is not None:
        values_out = _out(values_out, values, "values_out")
    tb = typed_temp_bytes(n, kb, vb, kind)
    if temp is None or temp.numel() < tb:
        temp = alloc_temp(tb, keys.device)
    _on_stream(stream, temp, keys_out, values_out)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(keys.device):
        check(lib.hrs_sort_typed(_ptr(temp), ctypes.byref(sz), _ptr(keys), _ptr(keys_out), _ptr(values),
                                 _ptr(values_out), n, kb, vb, kind, _stream(stream)), "hrs_sort_typed")
    return keys_out, (values_out if values is not None else None)


_KINDS = {"uint": 0, "int": 1, "float": 2}


def sort_records(records: torch.Tensor, key_bytes: int, value_bytes: int, *, key_first: bool = True,
                 kind: str = "uint", begin_bit: int = 0, end_bit: int | None = None, records_out=None, temp=None,
                 stream=None) -> torch.Tensor:
    """hrs_sort_records: stable sort of interleaved records (array of structs).
    `records` is a contiguous CUDA tensor whose bytes are n records of key_bytes +
    value_bytes each (e.g. a uint8 tensor of shape (n, R) or an int32 tensor of (n, R/4));
    the key is the first (key_first) or the last field.  Returns records_out (same shape)."""
    if not records.is_cuda or not records.is_contiguous():
        raise ValueError("records must be a contiguous CUDA tensor")
    rbytes = key_bytes + value_bytes
    total = records.numel() * records.element_size()
    if total % rbytes:
        raise ValueError(f"{total} bytes is not a whole number of {rbytes}-byte records")
    n = total // rbytes
    if end_bit is None:
        end_bit = 8 * key_bytes
    if records_out is None:
        records_out = torch.empty_like(records)
    elif records_out.numel() * records_out.element_size() != total or not records_out.is_cuda:
        raise ValueError("records_out must have the size of records")
    sz = ctypes.c_size_t(0)
    ko = 0 if key_first else value_bytes
    check(lib.hrs_sort_records(None, ctypes.byref(sz), None, None, n, key_bytes, value_bytes, ko, begin_bit,
                               end_bit, _KINDS[kind], None), "hrs_sort_records(size)")
    if temp is None or temp.numel() < sz.value:
        temp = alloc_temp(sz.value, records.device)
    _on_stream(stream, temp, records_out)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(records.device):
        check(lib.hrs_sort_records(_ptr(temp), ctypes.byref(sz), _ptr(records), _ptr(records_out), n, key_bytes,
                                   value_bytes, ko, begin_bit, end_bit, _KINDS[kind], _stream(stream)),
              "hrs_sort_records")
    return records_out


def get_stats(temp: torch.Tensor, stream=None) -> dict:
    """Statistics of the last sort that used `temp` (synchronises the stream)."""
    st = Stats()
    with torch.cuda.device(temp.device):
        check(lib.hrs_get_stats(_ptr(temp), ctypes.byref(st), _stream(stream)), "hrs_get_stats")
    return st.to_dict()


def digit_histogram(keys: torch.Tensor, lo_bit: int, hi_bit: int, *, temp: torch.Tensor | None = None,
                    stream=None) -> torch.Tensor:
    """2^(hi-lo) uint64 counts of digit bits [lo_bit, hi_bit) (device tensor)."""
    _check_tensor(keys, "keys")
    kb = _nbytes(keys, "keys")
    n = keys.numel()
    sz = ctypes.c_size_t(0)
    check(lib.hrs_digit_histogram(None, ctypes.byref(sz), None, n, kb, lo_bit, hi_bit, None, None),
          "hrs_digit_histogram(size query)")
    if temp is None or temp.numel() < sz.value:
        temp = alloc_temp(sz.value, keys.device)
    hist = torch.empty(1 << (hi_bit - lo_bit), dtype=torch.uint64, device=keys.device)
    _on_stream(stream, temp, hist)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(keys.device):
        check(lib.hrs_digit_histogram(_ptr(temp), ctypes.byref(sz), _ptr(keys), n, kb, lo_bit, hi_bit, _ptr(hist),
                                      _stream(stream)), "hrs_digit_histogram")
    return hist


def partition_pass(keys: torch.Tensor, values: torch.Tensor | None, lo_bit: int, hi_bit: int, *,
                   keys_out: torch.Tensor | None = None, values_out: torch.Tensor | None = None,
                   temp: torch.Tensor | None = None, stream=None):
    """One stable counting pass on digit bits [lo_bit, hi_bit): (keys_out, values_out, offsets[r+1])."""
    _check_tensor(keys, "keys")
    if keys.dtype in _TYPED_KEYS:
        raise TypeError("partition_pass takes unsigned keys (torch.uint32 / torch.uint64): a digit of a "
                        "signed or floating-point key is a digit of its order-preserving image (P:907-918); "
                        "map the keys first or use sort()")
    kb = _nbytes(keys, "keys")
    vb = 0
    if values is not None:
        _check_tensor(values, "values")
        vb = _nbytes(values, "values")
        if values.numel() != keys.numel() or values.device != keys.device:
            raise ValueError("keys and values differ in length or device")
    n = keys.numel()
    sz = ctypes.c_size_t(0)
    check(lib.hrs_partition_pass(None, ctypes.byref(sz), None, None, None, None, n, kb, vb, lo_bit, hi_bit, None,
                                 None), "hrs_partition_pass(size query)")
    if temp is None or temp.numel() < sz.value:
        temp = alloc_temp(sz.value, keys.device)
    keys_out = _out(keys_out, keys, "keys_out")
    if values is not None:
        values_out = _out(values_out, values, "values_out")
    offs = torch.empty((1 << (hi_bit - lo_bit)) + 1, dtype=torch.uint64, device=keys.device)
    _on_stream(stream, temp, keys_out, values_out, offs)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(keys.device):
        check(lib.hrs_partition_pass(_ptr(temp), ctypes.byref(sz), _ptr(keys), _ptr(keys_out), _ptr(values),
                                     _ptr(values_out), n, kb, vb, lo_bit, hi_bit, _ptr(offs), _stream(stream)),
              "hrs_partition_pass")
    return keys_out, (values_out if values is not None else None), offs


def copy_pieces(dst: torch.Tensor, src: torch.Tensor, pieces, stream=None) -> None:
    """hrs_copy_pieces: dst[d:d+c] = src[s:s+c] for every (s, d, c) in `pieces` (host list)."""
    _check_tensor(dst, "dst")
    _check_tensor(src, "src")
    if dst.dtype != src.dtype or dst.element_size() not in (4, 8):
        raise TypeError("copy_pieces takes two tensors of one 4- or 8-byte dtype")
    pcs = [(int(a), int(d), int(c)) for a, d, c in pieces if int(c) > 0]
    if not pcs:
        return
    for so, d, c in pcs:
        if so < 0 or d < 0 or so + c > src.numel() or d + c > dst.numel():
            raise ValueError("piece out of range")
    tab = (ctypes.c_uint64 * (3 * len(pcs)))(*[x for pc in pcs for x in pc])
    with torch.cuda.device(dst.device):
        check(lib.hrs_copy_pieces(_ptr(dst), _ptr(src), dst.element_size(), ctypes.cast(tab, ctypes.c_void_p),
                                  len(pcs), _stream(stream)),
              "hrs_copy_pieces")


def partition_pass_to(keys: torch.Tensor, values: torch.Tensor | None, lo_bit: int, hi_bit: int, dst_offsets,
                      key_windows, value_windows=None, *, temp: torch.Tensor | None = None, stream=None) -> None:
    """hrs_partition_pass_to: one stable counting pass on digit bits [lo_bit, hi_bit) whose
    digit-d records go to key_windows[w][o : o + count_d] (values likewise), with
    (w, o) = (dst_offsets[d] >> 48, dst_offsets[d] & (2^48 - 1)).  Windows are tensors
    (or raw device addresses, e.g. another GPU's buffer mapped over NVLink)."""
    _check_tensor(keys, "keys")
    kb = _nbytes(keys, "keys")
    vb = 0
    if values is not None:
        _check_tensor(values, "values")
        vb = _nbytes(values, "values")
    n = keys.numel()
    addr = lambda t: int(t) if isinstance(t, int) else t.data_ptr()  # noqa: E731
    kw = [addr(t) for t in key_windows]
    vw = [addr(t) for t in value_windows] if values is not None else [0] * len(kw)
    offs = [int(x) for x in dst_offsets]
    sz = ctypes.c_size_t(0)
    check(lib.hrs_partition_pass_to(None, ctypes.byref(sz), None, None, n, kb, vb, lo_bit, hi_bit, None, 0, None,
                                    None, None), "hrs_partition_pass_to(size query)")
    if temp is None or temp.numel() < sz.value:
        temp = alloc_temp(sz.value, keys.device)
    _on_stream(stream, temp)
    U = ctypes.c_uint64
    to = (U * len(offs))(*offs)
    tk = (U * len(kw))(*kw)
    tv = (U * len(vw))(*vw)
    sz = ctypes.c_size_t(temp.numel())
    with torch.cuda.device(keys.device):
        check(lib.hrs_partition_pass_to(_ptr(temp), ctypes.byref(sz), _ptr(keys), _ptr(values), n, kb, vb, lo_bit,
                                        hi_bit, ctypes.cast(to, ctypes.c_void_p), len(kw),
                                        ctypes.cast(tk, ctypes.c_void_p), ctypes.cast(tv, ctypes.c_void_p),
                                        _stream(stream)), "hrs_partition_pass_to")


def default_tuning(key_bytes: int, value_bytes: int) -> dict:
    t = Tuning()
    check(lib.hrs_default_tuning(key_bytes, value_bytes, ctypes.byref(t)), "hrs_default_tuning")
    return {f: getattr(t, f) for f, _ in Tuning._fields_}


def max_local_threshold(key_bytes: int, value_bytes: int) -> int:
    return lib.hrs_max_local_threshold(key_bytes, value_bytes)


def max_keys_per_tile(key_bytes: int, value_bytes: int) -> int:
    return lib.hrs_max_keys_per_tile(key_bytes, value_bytes)


def class_capacities() -> list:
    """Capacity of every local-sort size class of this build (hrs_class_capacity)."""
    from ._lib import HRS_NUM_CLASSES
    return [lib.hrs_class_capacity(c) for c in range(HRS_NUM_CLASSES)]


def profile_enable(on: bool = True) -> None:
    """Per-launch CUDA-event timing of this thread's library launches (see hrs.h)."""
    lib.hrs_profile_enable(1 if on else 0)


def profile_collect(max_records: int = 1 << 16) -> list:
    """[(kind, pass, ms)] of the launches since profile_enable; clears the list."""
    from ._lib import PROFILE_KINDS, ProfileRecord
    buf = (ProfileRecord * max_records)()
    k = lib.hrs_profile_collect(buf, max_records)
    return [(PROFILE_KINDS.get(r.kind, str(r.kind)), r.pass_, r.ms) for r in buf[:k]]


def launch_count() -> int:
    """Kernel launches this thread has enqueued through the library."""
    return lib.hrs_launch_count()
