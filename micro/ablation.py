"""The paper's ablation (Appendix B, Figs 11-14) rerun on B200: the hybrid sort
with and without tiny-bucket merging and with the size-class local sort vs a single local
configuration, for 32-bit keys, 32/32 pairs, 64-bit keys and 64/64 pairs over the entropy
sweep (uniform, AND-2/3/4).  2^28 records, inputs in HBM, CUDA events, median of 5.
    python micro/ablation.py [log2n]"""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import gen  # noqa: E402
import paper_1611_01137_b200 as hrs  # noqa: E402

lg = int(sys.argv[1]) if len(sys.argv) > 1 else 28
n = 1 << lg
VARIANTS = [("hybrid (default)", None), ("no merging", dict(merge_threshold=1)),
            ("single local config", dict(local_classes=1)),
            ("no merging + single config", dict(merge_threshold=1, local_classes=1))]
print(f"# ablation, n = 2^{lg}: ms per sort (records/s in G) -- fraction of the default's throughput")
for kbits, vbits in ((32, 0), (32, 32), (64, 0), (64, 64)):
    for dist in ("uniform", "and2", "and3", "and4"):
        k = gen.keys(n, kbits, dist, device="cuda")
        v = gen.values(n, vbits, "index", device="cuda") if vbits else None
        ko = torch.empty_like(k)
        vo = torch.empty_like(v) if v is not None else None
        row, base = [], None
        for name, tun in VARIANTS:
            t = dict(tun) if tun else None
            if t is not None and t.get("local_classes"):
                # the single configuration sorts every bucket with the largest local-sort CTA
                t["local_threshold"] = hrs.default_tuning(kbits // 8, vbits // 8)["local_threshold"]
            temp = torch.empty(hrs.temp_bytes(n, kbits // 8, vbits // 8, 0, kbits, t), dtype=torch.uint8, device="cuda")
            for _ in range(2):
                hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp, tuning=t)
            ms = []
            for _ in range(5):
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record()
                hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp, tuning=t)
                b.record()
                torch.cuda.synchronize()
                ms.append(a.elapsed_time(b))
            m = statistics.median(ms)
            base = base or m
            row.append(f"{name}: {m:.2f} ms ({n / m / 1e6:.1f} G) {base / m:.2f}")
            del temp
        print(f"k{kbits}/v{vbits} {dist:7s} | " + " | ".join(row), flush=True)
        del k, v, ko, vo
