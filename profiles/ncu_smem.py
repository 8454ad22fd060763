"""Per CUDA source line: shared-memory wavefronts (actual / ideal) and instructions, from an
`ncu --page source --csv --print-source cuda,sass` export.  Shows where bank conflicts are."""
import csv
import sys


def main(path, ntop=30):
    rows = list(csv.reader(open(path)))
    hi = next(i for i, r in enumerate(rows) if r and r[0] == "Line No")
    h = rows[hi]
    cols = {n: h.index(n) for n in ("Instructions Executed", "L1 Wavefronts Shared", "L1 Wavefronts Shared Ideal",
                                    "Warp Stall Sampling (All Samples)")}
    agg, cur = [], None
    for r in rows[hi + 1:]:
        if len(r) < len(h):
            continue
        if r[0] not in ("", "-"):
            cur = [r[0], r[1], 0.0, 0.0, 0.0, 0.0]
            agg.append(cur)
            continue
        if cur is None:
            continue
        for j, n in enumerate(cols):
            try:
                cur[2 + j] += float(r[cols[n]])
            except ValueError:
                pass
    tw = sum(a[3] for a in agg) or 1
    print(f"total smem wavefronts {tw:.0f}, ideal {sum(a[4] for a in agg):.0f}, instructions {sum(a[2] for a in agg):.0f}")
    for a in sorted(agg, key=lambda a: -a[3])[:ntop]:
        print(f"{a[3] / tw * 100:5.1f}% wf (x{a[3] / max(a[4], 1):4.2f} ideal) {a[2]:12.0f} inst  L{a[0]:>5} {a[1].strip()[:80]}")


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 30)
