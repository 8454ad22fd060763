"""CUDA IPC of device buffers between the processes of the distributed sort (one process per
GPU on a node: the opened address is the peer's memory over NVLink; two processes on one
GPU map the same device memory).  Used by the fused exchange (dist.py, exchange="fused")
to give hrs_partition_pass_to the peers' receive buffers as windows."""
from __future__ import annotations

_opened: dict = {}


def _check(err, what):
    code = err[0] if isinstance(err, tuple) else err
    if int(code) != 0:
        raise RuntimeError(f"{what} failed: {code}")


def export(t) -> tuple:
    """(IPC handle bytes of the allocation holding t, offset of t in it, device)."""
    from cuda.bindings import driver as drv
    from cuda.bindings import runtime as rt
    ptr = t.data_ptr()
    r = drv.cuMemGetAddressRange(ptr)
    _check(r, "cuMemGetAddressRange")
    base = int(r[1])
    r2 = rt.cudaIpcGetMemHandle(base)
    _check(r2, "cudaIpcGetMemHandle")
    return bytes(r2[1].reserved), ptr - base, t.device.index


def open(h: tuple) -> int:
    """The device address, in this process, of a buffer another process exported."""
    from cuda.bindings import runtime as rt
    raw, off, _dev = h
    if raw not in _opened:
        mh = rt.cudaIpcMemHandle_t()
        mh.reserved = raw
        r = rt.cudaIpcOpenMemHandle(mh, rt.cudaIpcMemLazyEnablePeerAccess)
        _check(r, "cudaIpcOpenMemHandle")
        _opened[raw] = int(r[1])
    return _opened[raw] + off
