"""Multi-process (world_size 2 and 3, gloo, CPU) tests of the distributed driver's host
logic: histogram gather, bucket assignment, split sizes, the all-to-all exchange and
the rank-order concatenation.  The local kernels are replaced by the CPU oracle (the
CUDA path of the same driver runs under NCCL on GPUs, see bench.py --gpus N)."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import gen
import oracle
from paper_1611_01137_b200 import dist as hdist


def _to_torch(a: np.ndarray, like: torch.Tensor) -> torch.Tensor:
    if like.dtype == torch.uint32:
        return torch.from_numpy(a.astype(np.uint32).view(np.int32).copy()).view(torch.uint32)
    return torch.from_numpy(a.astype(np.uint64).view(np.int64).copy()).view(torch.uint64)


class OracleOps:
    """Oracle-backed stand-ins for the CUDA kernels (test infrastructure only)."""

    def digit_histogram(self, keys, lo, hi):
        return torch.from_numpy(oracle.histogram(keys, lo, hi).astype(np.int64))

    def partition_pass(self, keys, vals, lo, hi):
        ko, vo, offs = oracle.partition_pass(keys, vals, lo, hi)
        return _to_torch(ko, keys), (_to_torch(vo, vals) if vals is not None else None), offs

    def sort(self, keys, vals, b, e):
        ko, vo = oracle.sort(keys, vals, b, e)
        return _to_torch(ko, keys), (_to_torch(vo, vals) if vals is not None else None)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n_per, kbits, dist_name, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        k = gen.keys(n_per, kbits, dist_name, start=rank * n_per)
        v = gen.values(n_per, 64, "index", start=rank * n_per)
        sorter = hdist.DistributedSorter(k, v, ops=OracleOps())
        ko, vo, off = sorter.step()
        parts = [None] * world
        dist.all_gather_object(parts, (off, oracle._u64(ko).tolist(), oracle._u64(vo).tolist(), sorter.last))
        if rank == 0:
            q.put(parts)
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,kbits,dist_name", [(2, 32, "uniform"), (2, 64, "and3"), (3, 32, "and4"),
                                                   (2, 32, "const")])
def test_distributed_sort_matches_global_oracle(world, kbits, dist_name):
    n_per = 3000
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n_per, kbits, dist_name, q)) for r in range(world)]
    for p in procs:
        p.start()
    parts = q.get(timeout=240)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    # global input in rank order, global index = rank * n_per + i (reading #17)
    gk = np.concatenate([oracle._u64(gen.keys(n_per, kbits, dist_name, start=r * n_per)) for r in range(world)])
    gv = np.arange(world * n_per, dtype=np.uint64)
    ek, ev = oracle.sort(gk, gv, 0, kbits)
    off = 0
    for rank, (o, ko, vo, last) in enumerate(parts):
        assert o == off, (rank, o, off)
        assert ko == ek[off:off + len(ko)].tolist()
        assert vo == ev[off:off + len(vo)].tolist()
        off += len(ko)
    assert off == world * n_per


def test_assignment_is_contiguous_and_balanced():
    hist = [10] * 256
    owner = hdist.assign_buckets(hist, 4)
    assert owner == sorted(owner) and owner[0] == 0 and owner[-1] == 3
    assert [owner.count(j) for j in range(4)] == [64, 64, 64, 64]
    # a single heavy bucket cannot be split at first-digit granularity
    hist = [0] * 100 + [1000] + [0] * 155
    owner = hdist.assign_buckets(hist, 8)
    assert owner == sorted(owner) and owner[100] == 0
    assert hdist.split_counts([hist], owner, 8)[0] == [1000] + [0] * 7
    send = hdist.split_counts([[1] * 256, [2] * 256], hdist.assign_buckets([3] * 256, 2), 2)
    assert send == [[128, 128], [256, 256]]
