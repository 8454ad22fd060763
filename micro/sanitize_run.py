"""Sorts for compute-sanitizer (memcheck / racecheck / synccheck): all six key/value type
pairs, uniform / AND-3 / constant keys, default tuning (one counting pass + local sorts at
2^16, two passes at 2^20) and small thresholds (deep recursion, merging, every local class),
each checked against the CPU oracle.  Usage: python micro/sanitize_run.py [log2n ...]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import gen  # noqa: E402
import oracle  # noqa: E402
import paper_1611_01137_b200 as hrs  # noqa: E402

sizes = [int(x) for x in sys.argv[1:]] or [16]
TYPES = [(32, 0), (32, 32), (32, 64), (64, 0), (64, 32), (64, 64)]
TUNINGS = [None, dict(local_threshold=300, merge_threshold=100, keys_per_tile=128)]
bad = 0
runs = 0
for lg in sizes:
    n = (1 << lg) + 7
    for kb, vb in TYPES:
        for dist in ("uniform", "and3", "const"):
            for tun in TUNINGS:
                k = gen.keys(n, kb, dist, seed=lg)
                v = gen.values(n, vb, "random", seed=lg) if vb else None
                ko, vo = hrs.sort(k.cuda(), v.cuda() if v is not None else None, tuning=tun)
                torch.cuda.synchronize()
                ek, ev = oracle.sort(k, v, 0, kb)
                ok = np.array_equal(oracle._u64(ko.cpu()), ek) and (v is None or np.array_equal(oracle._u64(vo.cpu()), ev))
                runs += 1
                if not ok:
                    bad += 1
                    print("MISMATCH", lg, kb, vb, dist, tun, flush=True)
    # typed keys and the building blocks once per size
    kf = gen.keys(n, 32, "uniform", seed=3).view(torch.float32)
    hrs.sort(kf.cuda())
    kk = gen.keys(n, 32, "and2", seed=3).cuda()
    hrs.digit_histogram(kk, 24, 32)
    hrs.partition_pass(kk, kk.clone(), 8, 16)
torch.cuda.synchronize()
print(f"sanitize_run: {runs} sorts, {bad} mismatches", flush=True)
sys.exit(1 if bad else 0)
