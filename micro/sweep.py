"""The paper's secondary experiments on B200, through the public API:
  size sweep    (Fig 7): n = 2^18 .. 2^28, uniform, 32/32 and 64/64;
  entropy sweep (Fig 6): 2^28 records, AND of m = 1..11 draws + constant.
Each point: median of 7 timed sorts (CUDA events) after 3 warm-ups, records/s, the
paper's sort rate n(K+V)/t and bytes_min / (t * measured copy peak) from the device
stats.  Prints one line per point; python micro/sweep.py [size|entropy] [kbits]"""
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import gen  # noqa: E402
import paper_1611_01137_b200 as hrs  # noqa: E402


def peak():
    try:
        return float(json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))["hbm_gbs"])
    except Exception:  # noqa: BLE001
        return 6650.0


def point(n, kbits, dist):
    k = gen.keys(n, kbits, dist, device="cuda")
    v = gen.values(n, kbits, "index", device="cuda")
    ko, vo = torch.empty_like(k), torch.empty_like(v)
    temp = torch.empty(hrs.temp_bytes(n, kbits // 8, kbits // 8), dtype=torch.uint8, device="cuda")
    for _ in range(3):
        hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp)
    ts = []
    for _ in range(7):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp)
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    t = statistics.median(ts)
    st = hrs.get_stats(temp)
    rec = 2 * kbits // 8
    frac = st["bytes_min"] / (t * 1e-3) / (peak() * 1e9)
    print(f"n=2^{n.bit_length() - 1:<2d} k{kbits}v{kbits} {dist:7s} {t:8.3f} ms  {n / t / 1e6:8.2f} G rec/s  "
          f"sort rate {n * rec / t / 1e6:7.1f} GB/s  passes {st['counting_passes']}  "
          f"B/rec {st['bytes_min'] / n:6.1f}  frac(measured peak) {frac:.3f}", flush=True)
    del k, v, ko, vo, temp
    torch.cuda.empty_cache()


if __name__ == "__main__":
    what = sys.argv[1] if len(sys.argv) > 1 else "size"
    kbits = int(sys.argv[2]) if len(sys.argv) > 2 else 32
    if what == "size":
        for lg in range(18, 29, 2):
            point(1 << lg, kbits, "uniform")
    else:
        for d in ["uniform"] + [f"and{m}" for m in range(2, 12)] + ["const"]:
            point(1 << 28, kbits, d)
