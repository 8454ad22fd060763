"""Multi-GPU stable sort: one process per GPU, torch.distributed (NCCL) for the exchange.

The MSD first digit is a key-range partition, so the sort shards with ONE exchange
step (the paper itself is single-GPU and scales out through a
host merge, which this replaces):

  1. every rank histograms the most-significant digit of its shard (libhrs kernel);
  2. all_gather of the 256-bin histograms (2 KiB per rank);
  3. a deterministic bucket -> rank assignment, identical on every rank: rank j owns
     the contiguous digit range whose global prefix starts in [j N/G, (j+1) N/G);
  4. one stable counting pass on that digit (libhrs kernel) groups the shard by
     destination, and all_to_all_single exchanges keys and values over NVLink;
  5. every rank sorts what it received with the single-GPU hybrid sort.  The
     received segments arrive in source-rank order, i.e. global input order, so the
     concatenation of the rank outputs is the unique stable sort of the global input
     (reading #17 in DESIGN.md: global index = rank-major).

The local operations are injected (`ops`): the product uses the CUDA library
(`CudaOps`); the CPU gloo tests inject an oracle-backed implementation to check the
host-side plumbing (assignment, split sizes, exchange order) without a GPU.
"""
from __future__ import annotations

import torch
import torch.distributed as dist

_SIGNED = {torch.uint32: torch.int32, torch.uint64: torch.int64}


def _bits(t: torch.Tensor) -> torch.Tensor:
    """Signed view with the same bits (collectives do not take unsigned dtypes)."""
    return t.view(_SIGNED[t.dtype]) if t.dtype in _SIGNED else t


class CudaOps:
    """The product's local operations: libhrs kernels through the C ABI."""

    def __init__(self):
        import paper_1611_01137_b200 as hrs
        self.hrs = hrs

    def digit_histogram(self, keys, lo, hi):
        return self.hrs.digit_histogram(keys, lo, hi)

    def partition_pass(self, keys, vals, lo, hi):
        return self.hrs.partition_pass(keys, vals, lo, hi)

    def sort(self, keys, vals, begin_bit, end_bit):
        return self.hrs.sort(keys, vals, begin_bit, end_bit)


def assign_buckets(global_hist: list[int], world: int) -> list[int]:
    """owner[b] for the 256 top-digit buckets: rank j owns the buckets whose global
    exclusive prefix lies in [j N / G, (j + 1) N / G) -- contiguous, monotone,
    deterministic (every rank computes the same list)."""
    n = sum(global_hist)
    owner = []
    run = 0
    for c in global_hist:
        owner.append(min(world - 1, (run * world) // n) if n else 0)
        run += c
    return owner


def split_counts(hists: list[list[int]], owner: list[int], world: int):
    """send[r][j] = records rank r sends to rank j (hists[r] = rank r's histogram)."""
    out = []
    for h in hists:
        row = [0] * world
        for b, c in enumerate(h):
            row[owner[b]] += c
        out.append(row)
    return out


class DistributedSorter:
    """Sorts the global array formed by concatenating every rank's (keys, vals) shard
    in rank order.  step() returns this rank's slice of the sorted output and its
    global offset."""

    def __init__(self, keys: torch.Tensor, vals: torch.Tensor | None = None, group=None, begin_bit: int = 0,
                 end_bit: int | None = None, ops=None):
        self.keys, self.vals, self.group = keys, vals, group
        self.kbits = 8 * keys.element_size()
        self.begin = begin_bit
        self.end = self.kbits if end_bit is None else end_bit
        self.ops = ops if ops is not None else CudaOps()
        self.world = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.last = {}

    def step(self):
        keys, vals = self.keys, self.vals
        world = self.world
        hi = self.end
        lo = max(self.begin, hi - 8)
        if hi == lo:  # empty bit range: the stable sort is the identity
            return keys.clone(), (vals.clone() if vals is not None else None), self._offset_identity()
        r = 1 << (hi - lo)
        # 1-2. first-digit histograms, gathered on every rank
        h = self.ops.digit_histogram(keys, lo, hi)
        gathered = torch.empty(world * r, dtype=torch.int64, device=h.device)
        dist.all_gather_into_tensor(gathered, _bits(h).contiguous(), group=self.group)
        hists = gathered.view(world, r).cpu().tolist()
        glob = [sum(col) for col in zip(*hists)]
        # 3. deterministic assignment of buckets to ranks
        owner = assign_buckets(glob, world)
        send = split_counts(hists, owner, world)
        recv = [send[src][self.rank] for src in range(world)]
        # 4. stable partition by destination (bucket order = destination order) + exchange
        kp, vp, _ = self.ops.partition_pass(keys, vals, lo, hi)
        rk = torch.empty(sum(recv), dtype=keys.dtype, device=keys.device)
        dist.all_to_all_single(_bits(rk), _bits(kp), output_split_sizes=recv,
                               input_split_sizes=send[self.rank], group=self.group)
        rv = None
        if vals is not None:
            rv = torch.empty(sum(recv), dtype=vals.dtype, device=vals.device)
            dist.all_to_all_single(_bits(rv), _bits(vp), output_split_sizes=recv,
                                   input_split_sizes=send[self.rank], group=self.group)
        # 5. local sort of the received records (source-rank order = global input order)
        ko, vo = self.ops.sort(rk, rv, self.begin, self.end)
        offset = sum(c for b, c in enumerate(glob) if owner[b] < self.rank)
        self.last = {"send": send[self.rank], "recv": recv, "owner": owner, "offset": offset,
                     "imbalance": max(sum(send[s][j] for s in range(world)) for j in range(world)) /
                     max(1, sum(glob) / world)}
        return ko, vo, offset

    def _offset_identity(self):
        n = torch.tensor([self.keys.numel()], dtype=torch.int64, device=self.keys.device)
        allv = torch.empty(self.world, dtype=torch.int64, device=n.device)
        dist.all_gather_into_tensor(allv, n, group=self.group)
        return int(allv[: self.rank].sum())


def sort(keys, vals=None, group=None, begin_bit: int = 0, end_bit: int | None = None):
    """hrs.dist.sort(keys, values, group) -> (keys_out, values_out, global_rank_offset)."""
    return DistributedSorter(keys, vals, group, begin_bit, end_bit).step()
