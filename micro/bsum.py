"""Summarise bench.py JSON lines: python micro/bsum.py gpurun_out/bench_c*.json"""
import json
import sys

for f in sys.argv[1:]:
    try:
        d = json.loads(open(f).read().strip().splitlines()[-1])
    except Exception as e:  # noqa: BLE001
        print(f, "unreadable", e)
        continue
    sr = d.get("sort_roofline", {})
    ks = d.get("kernels_ms_per_step", {})
    big = {k: v for k, v in ks.items() if v > 0.02}
    print(f"{d['config']['workload'][:40]:40s} {d['ms_per_step']:.3f} ms  frac {sr.get('frac', 0):.3f} "
          f"(8TB {sr.get('frac_of_8tbs', 0):.3f}) B/rec {sr.get('bytes_per_record', 0):.1f}  {big}")
