"""MSD hybrid-radix-sort bookkeeping, step by step in the paper's order -- TEST INFRASTRUCTURE.

Follows PAPER.md §4.1-4.2 and §4.5:
  * Fig 1 / P:430-456: a counting sort on the most-significant digit, then every
    sub-bucket is either partitioned again on the next digit or local-sorted; the
    sort ends when every key is sorted up to the least-significant digit or every
    bucket was local-sorted.
  * R1/R2: a bucket of size s is local-sorted iff s <= local_threshold
    (the paper's ∂ˆ), otherwise counting-sorted.
  * R3: after a bucket is partitioned, any sequence of its
    sub-buckets is merged while their total stays below merge_threshold (∂).
  * R4: a counting-sorted bucket of size s is cut into ceil(s/KPB) tiles.
  * Size classes [1,128], (128,256], (256,512], ....

Readings where the paper is silent:
  #3 digits are aligned to end_bit, the least-significant one may be narrower;
  #5 merging is greedy, left to right in digit order, strict "<", empty
     sub-buckets are skipped, a sub-bucket > ∂ˆ closes the current group;
  #6 a merged group (>= 2 non-empty sub-buckets) is local-sorted on bits
     [begin, hi_p), a single sub-bucket on [begin, lo_p);
  #7 after the last digit every sub-bucket is done;
  edge: n <= ∂ˆ means no counting pass, one local sort of [0, n) on [begin, end).

The sort permutation itself comes from numpy's stable argsort used as the
"stable partition" primitive; the arithmetic here is only the bookkeeping.
"""
from __future__ import annotations

from dataclasses import dataclass, field

import numpy as np


def digit_plan(begin_bit: int, end_bit: int):
    """[(lo_p, hi_p)] for p = 1..D, most-significant first (reading #3)."""
    out = []
    hi = end_bit
    while hi > begin_bit:
        lo = max(begin_bit, hi - 8)
        out.append((lo, hi))
        hi = lo
    return out


NUM_CLASSES = 8


def class_capacity(c: int) -> int:
    """Upper size of local-sort class c as P:562-566 gives it: [1,128], (128,256],
    (256,512], ... -- powers of two, 128 * 2^c."""
    return 128 << c


PAPER_CLASSES = tuple(class_capacity(c) for c in range(NUM_CLASSES))


def size_class(size: int, capacities=PAPER_CLASSES) -> int:
    """Smallest class whose capacity holds `size` records (capped at the last class).
    `capacities` is the class table (default: the paper's powers of two); a build whose
    tuning uses other boundaries (reading #20) passes its own table, which the
    classes then only rename -- the sort, pass and bucket structure do not depend on it."""
    c = 0
    while capacities[c] < size and c < len(capacities) - 1:
        c += 1
    return c


def classify_bucket(tot, last_digit: bool, local_threshold: int, merge_threshold: int):
    """Classify the sub-buckets of one partitioned bucket (digits in ascending order).

    Returns a list of ('done'|'count'|'local', [digits], size) in digit order.
    """
    out = []
    group: list[int] = []
    gsize = 0

    def close():
        nonlocal group, gsize
        if group:
            out.append(("local", group, gsize))
        group, gsize = [], 0

    for d, s in enumerate(int(x) for x in tot):
        if s == 0:
            continue
        if last_digit:
            out.append(("done", [d], s))
            continue
        if s > local_threshold:
            close()
            out.append(("count", [d], s))
            continue
        if group and gsize + s < merge_threshold:
            group.append(d)
            gsize += s
        else:
            close()
            group, gsize = [d], s
    close()
    return out


@dataclass
class MsdResult:
    keys: np.ndarray
    vals: np.ndarray | None
    counting_passes: int = 0
    recs_in_pass: list = field(default_factory=list)
    tiles_in_pass: list = field(default_factory=list)
    buckets_in_pass: list = field(default_factory=list)
    local_entries: list = field(default_factory=list)  # (offset, count, hi_bit, class, pass)
    merged_groups: int = 0
    skipped_in_pass: list = field(default_factory=list)  # S_p: records whose pass-p scatter is skipped

    @property
    def local_buckets(self):
        return len(self.local_entries)

    @property
    def local_recs(self):
        return sum(e[1] for e in self.local_entries)


def _sk(keys: np.ndarray, lo: int, hi: int) -> np.ndarray:
    w = hi - lo
    if w == 0:
        return np.zeros(keys.shape, dtype=np.uint64)
    mask = np.uint64((1 << w) - 1) if w < 64 else np.uint64(0xFFFFFFFFFFFFFFFF)
    return (keys >> np.uint64(lo)) & mask


def simulate_msd(keys, vals=None, begin_bit: int = 0, end_bit: int = 32,
                 local_threshold: int = 4096, merge_threshold: int = 3000,
                 keys_per_tile: int = 4096, class_capacities=PAPER_CLASSES) -> MsdResult:
    """Run the MSD hybrid sort on uint64 arrays; returns sorted data plus its structure.
    Local entries are labelled with their size class under `class_capacities`."""
    k = np.array(keys, dtype=np.uint64, copy=True)
    v = None if vals is None else np.array(vals, dtype=np.uint64, copy=True)
    n = k.size
    res = MsdResult(keys=k, vals=v)
    if n == 0 or begin_bit == end_bit:
        return res

    def local_sort(off, cnt, hi_bit, p):
        seg = slice(off, off + cnt)
        order = np.argsort(_sk(k[seg], begin_bit, hi_bit), kind="stable")
        k[seg] = k[seg][order]
        if v is not None:
            v[seg] = v[seg][order]
        res.local_entries.append((off, cnt, hi_bit, size_class(cnt, class_capacities), p))

    if n <= local_threshold:
        local_sort(0, n, end_bit, 0)
        return res

    plan = digit_plan(begin_bit, end_bit)
    # (offset, count, moved): `moved` -- some earlier pass scattered the bucket's records out
    # of the input buffer.  Reading #22: a bucket that never moved and whose
    # digit is the same for all its records is not scattered (a scatter would only copy it),
    # except in the last pass (whose output is the final result).
    buckets = [(0, n, False)]
    for p, (lo, hi) in enumerate(plan, start=1):
        if not buckets:
            break
        res.counting_passes = p
        res.recs_in_pass.append(sum(c for _, c, _ in buckets))
        res.tiles_in_pass.append(sum(-(-c // keys_per_tile) for _, c, _ in buckets))
        res.buckets_in_pass.append(len(buckets))
        res.skipped_in_pass.append(0)
        last = p == len(plan)
        nxt = []
        for off, cnt, moved in buckets:
            seg = slice(off, off + cnt)
            dig = _sk(k[seg], lo, hi)
            order = np.argsort(dig, kind="stable")  # the stable partition of this bucket
            k[seg] = k[seg][order]
            if v is not None:
                v[seg] = v[seg][order]
            tot = np.bincount(dig.astype(np.int64), minlength=1 << (hi - lo))
            starts = np.concatenate([[0], np.cumsum(tot)[:-1]]) + off
            skip = not last and not moved and int(np.count_nonzero(tot)) == 1
            if skip:
                res.skipped_in_pass[-1] += cnt
            for kind, ds, size in classify_bucket(tot, last, local_threshold, merge_threshold):
                start = int(starts[ds[0]])
                if kind == "count":
                    nxt.append((start, size, not skip))
                elif kind == "local":
                    if len(ds) >= 2:
                        res.merged_groups += 1
                    local_sort(start, size, hi if len(ds) >= 2 else lo, p)
        buckets = nxt
    return res


def bytes_min(res: MsdResult, key_bytes: int, value_bytes: int) -> int:
    """sum_p [R_p K + (R_p - S_p) 2(K+V)] + R_L * 2(K+V) -- every record of a
    pass is histogrammed, the records of skipped buckets (S_p, reading #22) are not moved."""
    rec = key_bytes + value_bytes
    return sum(r * key_bytes + (r - sk) * 2 * rec for r, sk in zip(res.recs_in_pass, res.skipped_in_pass)) + \
        res.local_recs * 2 * rec
