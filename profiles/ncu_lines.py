"""Aggregate an `ncu --page source --csv --print-source cuda,sass` export per CUDA source line:
instructions executed and warp-stall samples, top N lines."""
import csv
import sys


def main(path, ntop=30):
    rows = list(csv.reader(open(path)))
    hi = next(i for i, r in enumerate(rows) if r and r[0] == "Line No")
    h = rows[hi]
    ie = h.index("Instructions Executed")
    iS = h.index("Warp Stall Sampling (All Samples)")
    agg = []
    cur = None
    for r in rows[hi + 1:]:
        if len(r) < len(h):
            continue
        if r[0] not in ("", "-"):
            cur = [r[0], r[1], 0.0, 0.0]
            agg.append(cur)
            continue
        if cur is None:
            continue
        try:
            cur[2] += float(r[ie])
            cur[3] += float(r[iS])
        except ValueError:
            pass
    ti = sum(a[2] for a in agg) or 1
    ts = sum(a[3] for a in agg) or 1
    print(f"total warp instructions {ti:.0f}")
    for a in sorted(agg, key=lambda a: -a[2])[:ntop]:
        print(f"{a[2] / ti * 100:5.1f}% inst {a[3] / ts * 100:5.1f}% stall  L{a[0]:>5} {a[1].strip()[:90]}")


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 30)
