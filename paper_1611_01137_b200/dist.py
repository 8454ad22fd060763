"""Multi-GPU stable sort: one process per GPU, torch.distributed (NCCL) for the exchange.

The MSD first digit is a key-range partition, so the sort shards with ONE exchange
step (the paper itself is single-GPU and scales out through a
host merge, which this replaces):

  1. every rank histograms the most-significant digit of its shard (libhrs kernel);
  2. all_gather of the 256-bin histograms (2 KiB per rank);
  3. one stable counting pass on that digit (libhrs kernel) groups the shard by bucket;
     rank j receives exactly the global sorted positions [j N/G, (j+1) N/G) (SURVEY
     §8(f) N1, skew-robust splitting): only the buckets that contain a boundary j N/G
     are refined, digit by digit, with the same stable counting pass on their local
     sub-ranges and an all_gather of their sub-bucket histograms; at full key
     resolution a boundary lies inside a run of equal keys, which is split by global
     index (rank-major, reading #17).  Every rank then knows every rank's split
     positions, so the send/receive counts need no further exchange;
  4. all_to_all_single exchanges keys and values over NVLink;
  5. every rank sorts what it received with the single-GPU hybrid sort.  The
     received segments arrive in source-rank order, i.e. global input order, so the
     concatenation of the rank outputs is the unique stable sort of the global input
     (reading #17 in DESIGN.md: global index = rank-major).

The local operations are injected (`ops`): the product uses the CUDA library
(`CudaOps`); the CPU gloo tests inject an oracle-backed implementation to check the
host-side plumbing (split positions, split sizes, exchange order) without a GPU.
"""
from __future__ import annotations

import torch
import torch.distributed as dist

_SIGNED = {torch.uint32: torch.int32, torch.uint64: torch.int64}


def _bits(t: torch.Tensor) -> torch.Tensor:
    """Signed view with the same bits (collectives do not take unsigned dtypes)."""
    return t.view(_SIGNED[t.dtype]) if t.dtype in _SIGNED else t


def _host_staged(group, t: torch.Tensor) -> bool:
    """gloo cannot run these collectives on CUDA tensors: stage them through host memory
    (used by the single-GPU multi-process tests; NCCL takes device tensors directly)."""
    return t.is_cuda and dist.get_backend(group) == "gloo"


def _all_gather(out: torch.Tensor, inp: torch.Tensor, group) -> None:
    if _host_staged(group, inp):
        o = out.cpu()
        dist.all_gather_into_tensor(o, inp.cpu(), group=group)
        out.copy_(o)
    else:
        dist.all_gather_into_tensor(out, inp, group=group)


def _all_to_all(out: torch.Tensor, inp: torch.Tensor, out_splits, in_splits, group) -> None:
    if _host_staged(group, inp):
        o = out.cpu()
        dist.all_to_all_single(o, inp.cpu(), output_split_sizes=out_splits, input_split_sizes=in_splits, group=group)
        out.copy_(o)
    else:
        dist.all_to_all_single(out, inp, output_split_sizes=out_splits, input_split_sizes=in_splits, group=group)


class CudaOps:
    """The product's local operations: libhrs kernels through the C ABI."""

    def __init__(self):
        import paper_1611_01137_b200 as hrs
        self.hrs = hrs

    def digit_histogram(self, keys, lo, hi):
        return self.hrs.digit_histogram(keys, lo, hi)

    def partition_pass(self, keys, vals, lo, hi):
        return self.hrs.partition_pass(keys, vals, lo, hi)

    def partition_into(self, keys, vals, lo, hi, keys_out, vals_out):
        """Stable counting pass of keys (vals) into keys_out (vals_out); returns the
        sub-bucket offsets (r + 1 entries) on the host."""
        _, _, offs = self.hrs.partition_pass(keys, vals, lo, hi, keys_out=keys_out, values_out=vals_out)
        return offs.cpu().tolist()

    def sort(self, keys, vals, begin_bit, end_bit):
        return self.hrs.sort(keys, vals, begin_bit, end_bit)

    def copy_pieces(self, dst, src, pieces):
        self.hrs.copy_pieces(dst, src, pieces)

    def partition_pass_to(self, keys, vals, lo, hi, offsets, key_windows, value_windows):
        self.hrs.partition_pass_to(keys, vals, lo, hi, offsets, key_windows, value_windows)

    def sort_grouped_into(self, keys, vals, first_hist, begin_bit, end_bit, keys_out, vals_out, temp_holder):
        """hrs_sort_grouped into caller buffers (the input is grouped by its first digit)."""
        self._temp_for(keys, vals, begin_bit, end_bit, temp_holder)
        return self.hrs.sort_grouped(keys, vals, first_hist, begin_bit, end_bit, keys_out=keys_out,
                                     values_out=vals_out, temp=temp_holder[0])

    def _temp_for(self, keys, vals, begin_bit, end_bit, temp_holder):
        kb, vb = keys.element_size(), (vals.element_size() if vals is not None else 0)
        need = self.hrs.temp_bytes(keys.numel(), kb, vb, begin_bit, end_bit)
        if temp_holder[0] is None or temp_holder[0].numel() < need:
            temp_holder[0] = None
            temp_holder[0] = self.hrs.alloc_temp(need, keys.device)

    def sort_into(self, keys, vals, begin_bit, end_bit, keys_out, vals_out, temp_holder):
        """Sort into caller buffers with a temp kept across calls (temp_holder: a one-element
        list holding the temp tensor or None): no allocation on the step's critical path."""
        self._temp_for(keys, vals, begin_bit, end_bit, temp_holder)
        return self.hrs.sort(keys, vals, begin_bit, end_bit, keys_out=keys_out, values_out=vals_out,
                             temp=temp_holder[0])


class DistributedSorter:
    """Sorts the global array formed by concatenating every rank's (keys, vals) shard
    in rank order.  step() returns this rank's slice of the sorted output and its
    global offset."""

    def __init__(self, keys: torch.Tensor, vals: torch.Tensor | None = None, group=None, begin_bit: int = 0,
                 end_bit: int | None = None, ops=None, exchange: str = "grouped"):
        self.keys, self.vals, self.group = keys, vals, group
        self.kbits = 8 * keys.element_size()
        self.begin = begin_bit
        self.end = self.kbits if end_bit is None else end_bit
        self.ops = ops if ops is not None else CudaOps()
        if exchange not in ("grouped", "a2a", "fused"):
            raise ValueError(exchange)
        # "grouped": bucket-major point-to-point exchange, the receiver skips the first pass;
        # "a2a": one all_to_all_single per array, the receiver sorts from the first digit;
        # "fused": the partition scatter stores every bucket a single rank owns straight into
        #   that rank's receive buffer (mapped with CUDA IPC: NVLink peer memory on a node),
        #   only the buckets a rank boundary cuts are staged, refined and sent
        self.exchange = exchange
        self._windows_cache = None
        self.world = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.last = {}
        # time_exchange: CUDA events around step 4 (the all-to-all) on the current stream,
        # so bench.py can report the exchange against NVLink bandwidth
        self.time_exchange = False
        self.exchange_events = None
        # buffers kept across steps (memory at C5 scale): the partition output
        # (= send buffer, later the local sort's output), the receive buffer (= refinement
        # scratch before the exchange) and the local sort's temp
        self._kp = self._vp = None
        self._rk = self._rv = None
        self._temp = [None]

    def _send_buffers(self, n):
        if self._kp is None or self._kp.numel() != n:
            self._kp = self._vp = None
            self._kp = torch.empty_like(self.keys)
            self._vp = torch.empty_like(self.vals) if self.vals is not None else None
        return self._kp, self._vp

    def _recv_buffers(self, cap):
        if self._rk is None or self._rk.numel() < cap:
            self._rk = self._rv = None
            self._rk = torch.empty(cap, dtype=self.keys.dtype, device=self.keys.device)
            self._rv = (torch.empty(cap, dtype=self.vals.dtype, device=self.vals.device)
                        if self.vals is not None else None)
        return self._rk, self._rv

    def digits(self):
        """The (lo, hi) bit ranges of the 8-bit digits, most significant first."""
        out, hi = [], self.end
        while hi > self.begin:
            lo = max(self.begin, hi - 8)
            out.append((lo, hi))
            hi = lo
        return out

    def step(self):
        keys, vals = self.keys, self.vals
        world, me = self.world, self.rank
        if self.end == self.begin:  # empty bit range: the stable sort is the identity
            return keys.clone(), (vals.clone() if vals is not None else None), self._offset_identity()
        digits = self.digits()
        fused = self.exchange == "fused"
        # 1-3a. first-digit partition of the whole shard; its histogram, gathered
        kp, vp = self._send_buffers(keys.numel())
        lo, hi = digits[0]
        if fused:  # histogram first: the fused partition needs every rank's counts
            h = self.ops.digit_histogram(keys, lo, hi)
            hists = self._gather([[int(x) for x in h.view(torch.int64).cpu().tolist()]])[0]
        else:
            offs = self.ops.partition_into(keys, vals, lo, hi, kp, vp)
            hists = self._gather([[offs[b + 1] - offs[b] for b in range(len(offs) - 1)]])[0]  # [rank][bucket]
        N = sum(sum(h) for h in hists)
        cap = max((j + 1) * N // world - j * N // world for j in range(world))  # largest receive
        rk_all, rv_all = self._recv_buffers(cap)
        boundary = None
        if fused:
            boundary = self._fused_partition(keys, vals, hists, N, lo, hi, kp, vp, rk_all, rv_all)
        # split[j][r]: local position on rank r of global sorted position t_j = j N / G
        split = [[0] * world for _ in range(world + 1)]
        split[world] = [sum(h) for h in hists]
        todo = []  # boundaries inside a segment: (j, t_j, level, g0, starts[r], counts[r])
        for j in range(1, world):
            self._place(j, j * N // world, 0, 0, [0] * world, hists, split, todo)
        # 3b. refine the segments that contain a boundary, one digit at a time
        scratch_k = scratch_v = None
        levels = 0  # digits below the first that some boundary needed
        for level in range(1, len(digits)):
            if not todo:
                break
            levels = level
            if scratch_k is None:
                # the receive buffer is not in use before the exchange: it is the scratch of
                # the refinement passes (a refined sub-range larger than it gets its own)
                big = max(it[5][me] for it in todo)
                if big <= rk_all.numel() and not fused:  # (fused: peers are writing the receive buffer)
                    scratch_k, scratch_v = rk_all, rv_all
                else:
                    scratch_k = torch.empty(big, dtype=kp.dtype, device=kp.device)
                    scratch_v = torch.empty(big, dtype=vp.dtype, device=vp.device) if vp is not None else None
            lo, hi = digits[level]
            segs = []  # distinct segments (several boundaries may share one)
            for item in todo:
                if not segs or segs[-1][0] != (item[3], tuple(item[4])):
                    segs.append(((item[3], tuple(item[4])), item[4], item[5]))
            local = []
            for _, starts, counts in segs:
                a, c = starts[me], counts[me]
                if c:
                    sub = self.ops.partition_into(kp[a:a + c], vp[a:a + c] if vp is not None else None, lo, hi,
                                                  scratch_k[:c], scratch_v[:c] if vp is not None else None)
                    kp[a:a + c].copy_(scratch_k[:c])
                    if vp is not None:
                        vp[a:a + c].copy_(scratch_v[:c])
                    local.append([sub[b + 1] - sub[b] for b in range(len(sub) - 1)])
                else:
                    local.append([0] * (1 << (hi - lo)))
            seg_hists = self._gather(local)  # [seg][rank][sub-bucket]
            nxt = []
            for item in todo:
                k = next(i for i, sg in enumerate(segs) if sg[0] == (item[3], tuple(item[4])))
                self._place(item[0], item[1], level, item[3], item[4], seg_hists[k], split, nxt)
            todo = nxt
        # 3c. boundaries still inside a segment after the last digit: equal keys, split by
        # global index (rank-major, each rank's run in local index order)
        for j, t, _, g0, starts, counts in todo:
            run = g0
            for r in range(world):
                split[j][r] = starts[r] + min(counts[r], max(0, t - run))
                run += counts[r]
        send = [[split[j + 1][r] - split[j][r] for j in range(world)] for r in range(world)]
        recv = [send[src][me] for src in range(world)]
        m = sum(recv)
        rk = rk_all[:m]
        rv = rv_all[:m] if vals is not None else None
        grouped = self.exchange in ("grouped", "fused") and len(digits) >= 1
        if grouped:
            sends, recvs, rhist = self._grouped_plan(hists, split)
            if fused:
                # the fused scatter already stored every bucket that one rank owns; what is
                # left are the pieces of the (at most G - 1) buckets a rank boundary cuts,
                # which were staged locally and refined.  Every rank's stores must be done
                # before any receiver reads its buffer.
                sends = [x for x in sends if boundary[x[4]]]
                recvs = [x for x in recvs if boundary[x[3]]]
                self._barrier_after_device_work()
        ev = None
        if self.time_exchange and keys.is_cuda:
            ev = (torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
            ev[0].record()
        if grouped:
            # 4. bucket-major exchange: every (source, first-digit bucket) piece lands at its
            # place in the receiver's buffer -- bucket b's pieces from sources 0..G-1 in rank
            # order -- so the received records are grouped by the first digit and, within a
            # bucket, in global input order (reading #17)
            self._p2p(rk, kp, sends, recvs)
            if vals is not None:
                self._p2p(rv, vp, sends, recvs)
        else:
            # 4. all-to-all (every source's segment in source-rank order)
            _all_to_all(_bits(rk), _bits(kp), recv, send[me], self.group)
            if vals is not None:
                _all_to_all(_bits(rv), _bits(vp), recv, send[me], self.group)
        if ev is not None:
            ev[1].record()
        self.exchange_events = ev
        # 5. local sort of the received records, into the send buffers (dead after the
        # exchange) when they are large enough; a grouped receive buffer starts at the
        # second digit (hrs_sort_grouped: the first pass is already done by the exchange)
        outk = kp[:m] if m <= kp.numel() else None
        outv = (vp[:m] if vp is not None else None) if outk is not None else None
        if grouped and hasattr(self.ops, "sort_grouped_into") and outk is not None:
            ko, vo = self.ops.sort_grouped_into(rk, rv, rhist, self.begin, self.end, outk, outv, self._temp)
        elif hasattr(self.ops, "sort_into") and outk is not None:
            ko, vo = self.ops.sort_into(rk, rv, self.begin, self.end, outk, outv, self._temp)
        else:
            ko, vo = self.ops.sort(rk, rv, self.begin, self.end)
        offset = me * N // world
        self.last = {"send": send[me], "recv": recv, "offset": offset, "refine_levels": levels,
                     "imbalance": max(sum(send[s][j] for s in range(world)) for j in range(world)) /
                     max(1, N / world)}
        return ko, vo, offset

    def _grouped_plan(self, hists, split):
        """Pieces of the bucket-major exchange.  Rank r's partition output holds bucket b at
        [O_r(b), O_r(b+1)) (O_r = prefix of hists[r]); it sends [split[j][r], split[j+1][r])
        to rank j.  Receiver j stores, for every bucket b in ascending order, the pieces of
        sources 0..G-1 in rank order.  Returns this rank's sends [(peer, src_off, len,
        dst_off)], receives [(peer, dst_off, len)] (both in bucket order per peer, so the
        messages of a pair match in issue order) and the received first-digit histogram."""
        import numpy as np
        world, me = self.world, self.rank
        H = np.asarray(hists, dtype=np.int64)                 # [rank][bucket]
        R = H.shape[1]
        O = np.zeros((world, R + 1), dtype=np.int64)
        O[:, 1:] = np.cumsum(H, axis=1)                       # bucket starts per rank
        S = np.asarray(split, dtype=np.int64)                 # [j][rank] split positions
        # piece (j, b, r) = [max(S[j][r], O[r][b]), min(S[j+1][r], O[r][b+1]))
        a = np.maximum(S[:-1, None, :], O.T[None, :-1, :])    # [j][b][r]
        z = np.minimum(S[1:, None, :], O.T[None, 1:, :])
        ln = np.maximum(z - a, 0)
        dst = np.cumsum(ln.reshape(world, -1), axis=1).reshape(ln.shape) - ln  # receiver offsets, (b, r)-major
        sends = [(int(j), int(a[j, b, me]), int(ln[j, b, me]), int(dst[j, b, me]), int(b))
                 for j, b in zip(*np.nonzero(ln[:, :, me]))]
        recvs = [(int(r), int(dst[me, b, r]), int(ln[me, b, r]), int(b)) for b, r in zip(*np.nonzero(ln[me]))]
        rhist = ln[me].sum(axis=1).tolist()
        return sends, recvs, rhist

    def _p2p(self, rbuf, sbuf, sends, recvs):
        """The pieces as one batch of point-to-point messages (NCCL groups them; NVLink),
        this rank's own pieces as device copies (one launch).  With gloo (tests) the
        messages go through host copies and only the received ranges are copied back."""
        me = self.rank
        staged = _host_staged(self.group, sbuf)
        own = []
        for peer, a, ln, d, *_ in sends:
            if peer == me:
                if own and own[-1][0] + own[-1][2] == a and own[-1][1] + own[-1][2] == d:
                    own[-1] = (own[-1][0], own[-1][1], own[-1][2] + ln)  # contiguous on both sides
                else:
                    own.append((a, d, ln))
        if own:
            if hasattr(self.ops, "copy_pieces"):
                self.ops.copy_pieces(_bits(rbuf), _bits(sbuf), own)
            else:
                for a, d, ln in own:
                    _bits(rbuf)[d:d + ln].copy_(_bits(sbuf)[a:a + ln])
        peer_sends = [x for x in sends if x[0] != me]
        peer_recvs = [x for x in recvs if x[0] != me]
        if not peer_sends and not peer_recvs:
            return
        sbv = _bits(sbuf.cpu() if staged else sbuf)
        rbv = _bits(torch.empty_like(rbuf, device="cpu")) if staged else _bits(rbuf)
        ops = [dist.P2POp(dist.isend, sbv[a:a + ln], peer, self.group) for peer, a, ln, d, *_ in peer_sends]
        ops += [dist.P2POp(dist.irecv, rbv[d:d + ln], peer, self.group) for peer, d, ln, *_ in peer_recvs]
        for req in dist.batch_isend_irecv(ops):
            req.wait()
        if staged:
            for peer, d, ln, *_ in peer_recvs:
                _bits(rbuf)[d:d + ln].copy_(rbv[d:d + ln])

    def _fused_partition(self, keys, vals, hists, N, lo, hi, kp, vp, rk_all, rv_all):
        """The fused exchange's partition (hrs_partition_pass_to): bucket b that lies inside
        rank j's range [t_j, t_{j+1}) goes to j's receive buffer at its bucket-major place
        (C[b] - t_j + the counts of b on ranks before this one); a bucket that a boundary t_j
        cuts goes to this rank's staging buffer at its partitioned place.  Returns the
        boundary flags per bucket."""
        import numpy as np
        world, me = self.world, self.rank
        H = np.asarray(hists, dtype=np.int64)
        R = H.shape[1]
        tot = H.sum(axis=0)
        C = np.concatenate([[0], np.cumsum(tot)])
        t = np.array([j * N // world for j in range(world + 1)], dtype=np.int64)
        before = np.concatenate([np.zeros((1, R), dtype=np.int64), np.cumsum(H, axis=0)])[me]  # ranks < me
        O = np.concatenate([[0], np.cumsum(H[me])])
        boundary = [False] * R
        offs = [0] * R
        for b in range(R):
            if tot[b] == 0:
                continue
            j = int(np.searchsorted(t, C[b], side="right") - 1)  # t_j <= C[b] < t_{j+1}
            j = min(j, world - 1)
            if C[b + 1] > t[j + 1]:  # a rank boundary cuts the bucket
                boundary[b] = True
                offs[b] = (world << 48) | int(O[b])
            else:
                offs[b] = (j << 48) | int(C[b] - t[j] + before[b])
        kw, vw = self._windows(rk_all, rv_all)
        # every receiver is done with its buffer (the previous step's local sort read it)
        self._barrier_after_device_work()
        self.ops.partition_pass_to(keys, vals, lo, hi, offs, kw + [kp.data_ptr()],
                                   (vw + [vp.data_ptr()]) if vals is not None else None)
        return boundary

    def _windows(self, rk_all, rv_all):
        """Device addresses of every rank's receive buffers in this process: our own, and the
        peers' opened through CUDA IPC (exchanged once per buffer)."""
        key = (rk_all.data_ptr(), rv_all.data_ptr() if rv_all is not None else 0)
        if self._windows_cache is None or self._windows_cache[0] != key:
            from . import ipc
            mine = (ipc.export(rk_all), ipc.export(rv_all) if rv_all is not None else None)
            allh = [None] * self.world
            dist.all_gather_object(allh, mine, group=self.group)
            kw, vw = [], []
            for r, (hk, hv) in enumerate(allh):
                if r == self.rank:
                    kw.append(rk_all.data_ptr())
                    vw.append(rv_all.data_ptr() if rv_all is not None else 0)
                else:
                    kw.append(ipc.open(hk))
                    vw.append(ipc.open(hv) if hv is not None else 0)
            self._windows_cache = (key, kw, vw)
        return list(self._windows_cache[1]), list(self._windows_cache[2])

    def _barrier_after_device_work(self):
        """Every rank's device work so far (the fused stores into peers' buffers) is done
        before any rank goes on."""
        if self.keys.is_cuda:
            torch.cuda.current_stream().synchronize()
        if self.world > 1:
            dist.barrier(group=self.group)

    def _gather(self, rows):
        """all_gather of this rank's histogram rows ([k][r] ints) -> [k][rank][r]."""
        k, r = len(rows), len(rows[0])
        mine = torch.tensor(rows, dtype=torch.int64).reshape(-1)
        if self.keys.is_cuda:
            mine = mine.to(self.keys.device)
        allv = torch.empty(self.world * k * r, dtype=torch.int64, device=mine.device)
        _all_gather(allv, mine, self.group)
        a = allv.view(self.world, k, r).cpu().tolist()
        return [[a[q][i] for q in range(self.world)] for i in range(k)]

    def _place(self, j, t, level, g0, starts, hists, split, todo):
        """Global position t falls in the segment whose sub-buckets have per-rank sizes
        hists[rank][b] (global base g0, local starts[rank]): record its local split
        position on every rank if t is a sub-bucket edge, else queue the sub-bucket."""
        world = self.world
        base = g0
        local = list(starts)
        for b in range(len(hists[0])):
            tot = sum(h[b] for h in hists)
            if t < base + tot:
                if t == base:
                    break
                todo.append((j, t, level + 1, base, list(local), [h[b] for h in hists]))
                return
            base += tot
            for r in range(world):
                local[r] += hists[r][b]
        split[j] = local
    def _offset_identity(self):
        n = torch.tensor([self.keys.numel()], dtype=torch.int64, device=self.keys.device)
        allv = torch.empty(self.world, dtype=torch.int64, device=n.device)
        _all_gather(allv, n, self.group)
        return int(allv[: self.rank].sum())


def sort(keys, vals=None, group=None, begin_bit: int = 0, end_bit: int | None = None, exchange: str = "grouped"):
    """hrs.dist.sort(keys, values, group) -> (keys_out, values_out, global_rank_offset)."""
    return DistributedSorter(keys, vals, group, begin_bit, end_bit, exchange=exchange).step()
