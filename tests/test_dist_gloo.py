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

    def partition_into(self, keys, vals, lo, hi, keys_out, vals_out):
        ko, vo, offs = oracle.partition_pass(keys, vals, lo, hi)
        keys_out.copy_(_to_torch(ko, keys))
        if vals is not None:
            vals_out.copy_(_to_torch(vo, vals))
        return [int(x) for x in offs]

    def sort(self, keys, vals, b, e):
        ko, vo = oracle.sort(keys, vals, b, e)
        return _to_torch(ko, keys), (_to_torch(vo, vals) if vals is not None else None)

    def sort_grouped_into(self, keys, vals, first_hist, b, e, keys_out, vals_out, temp_holder):
        """The bucket-major exchange must deliver the records grouped by their first digit
        with exactly this histogram (hrs_sort_grouped's precondition): checked, then sorted."""
        lo = max(b, e - 8)
        dig = (oracle._u64(keys) >> np.uint64(lo)) & np.uint64((1 << (e - lo)) - 1)
        assert bool(np.all(dig[1:] >= dig[:-1])), "receive buffer not grouped by the first digit"
        assert np.bincount(dig.astype(np.int64), minlength=len(first_hist)).tolist() == list(first_hist)
        self.grouped_calls = getattr(self, "grouped_calls", 0) + 1
        return self.sort_into(keys, vals, b, e, keys_out, vals_out, temp_holder)

    def sort_into(self, keys, vals, b, e, keys_out, vals_out, temp_holder):
        """Into the driver's reused buffers (the send buffer), as the CUDA path does."""
        ko, vo = self.sort(keys, vals, b, e)
        keys_out.copy_(ko)
        if vals is not None:
            vals_out.copy_(vo)
        temp_holder[0] = "used"
        return keys_out, vals_out


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n_per, kbits, dist_name, q, exchange="grouped"):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        k = gen.keys(n_per, kbits, dist_name, start=rank * n_per)
        v = gen.values(n_per, 64, "index", start=rank * n_per)
        ops = OracleOps()
        sorter = hdist.DistributedSorter(k, v, ops=ops, exchange=exchange)
        ko, vo, off = sorter.step()
        ko = ko.clone()
        # a second step reuses every buffer (send / receive / temp) and must give the same
        ko2, vo2, off2 = sorter.step()
        assert off2 == off and torch.equal(ko2.view(torch.int64 if kbits == 64 else torch.int32),
                                           ko.view(torch.int64 if kbits == 64 else torch.int32))
        assert sorter._temp[0] == "used" and ko2.data_ptr() == sorter._kp.data_ptr()
        assert getattr(ops, "grouped_calls", 0) == (2 if exchange == "grouped" else 0)
        parts = [None] * world
        dist.all_gather_object(parts, (off, oracle._u64(ko).tolist(), oracle._u64(vo).tolist(), sorter.last))
        if rank == 0:
            q.put(parts)
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,kbits,dist_name,exchange", [(2, 32, "uniform", "grouped"), (2, 64, "and3", "grouped"),
                                                            (3, 32, "and4", "grouped"), (2, 32, "const", "grouped"),
                                                            (4, 32, "and4", "grouped"), (3, 64, "const", "grouped"),
                                                            (4, 64, "uniform", "grouped"), (3, 32, "and3", "a2a"),
                                                            (2, 64, "uniform", "a2a")])
def test_distributed_sort_matches_global_oracle(world, kbits, dist_name, exchange):
    """The rank outputs concatenate to the global stable sort, and every rank holds
    exactly its N/G share whatever the skew (exact splitting)."""
    n_per = 3000
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n_per, kbits, dist_name, q, exchange))
             for r in range(world)]
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
    N = world * n_per
    for rank, (o, ko, vo, last) in enumerate(parts):
        assert o == off, (rank, o, off)
        assert len(ko) == (rank + 1) * N // world - rank * N // world, (rank, len(ko))
        assert last["imbalance"] <= 1.0 + world / N
        assert ko == ek[off:off + len(ko)].tolist()
        assert vo == ev[off:off + len(vo)].tolist()
        off += len(ko)
    assert off == world * n_per


def test_split_positions_by_global_index():
    """_place / the final tie split on hand-made histograms (no processes)."""
    class S(hdist.DistributedSorter):
        def __init__(self, world):
            self.world, self.rank = world, 0
    s = S(3)
    # 2 ranks x 3 buckets: sizes [[2,0,4],[1,3,0]] -> global [3,3,4], N = 10
    hists = [[2, 0, 4], [1, 3, 0]]
    s.world = 2
    split = [[0, 0] for _ in range(3)]
    todo = []
    s._place(1, 3, 0, 0, [0, 0], hists, split, todo)  # t = 3: edge of bucket 1
    assert split[1] == [2, 1] and not todo
    s._place(1, 5, 0, 0, [0, 0], hists, split, todo)  # t = 5: inside bucket 1 (3..6)
    assert todo == [(1, 5, 1, 3, [2, 1], [0, 3])]
