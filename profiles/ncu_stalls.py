"""Per-instruction stall attribution from `ncu --page source --csv --print-source sass`:
kernel-wide stall-reason totals, then the top instructions with their dominant reasons and
the instructions just before them (a stall is charged to the instruction that waits)."""
import csv
import sys


def main(path, ntop=20):
    rows = list(csv.reader(open(path, encoding="utf-8", errors="replace")))
    hi = next(i for i, r in enumerate(rows) if "Source" in r and "Address" in r)
    h = rows[hi]
    data = [r for r in rows[hi + 1:] if len(r) == len(h) and r[0].startswith("0x")]
    seen, uniq = set(), []
    for r in data:
        if r[0] not in seen:
            seen.add(r[0])
            uniq.append(r)
    data = uniq
    f = lambda x: float(x) if x not in ("", None) else 0.0
    sc = [i for i, n in enumerate(h) if n.startswith("stall_") and "Not Issued" not in n]
    tot = {h[i]: sum(f(r[i]) for r in data) for i in sc}
    alls = sum(tot.values()) or 1
    print("stall totals:", ", ".join(f"{k[6:]}={v / alls * 100:.1f}%" for k, v in sorted(tot.items(), key=lambda x: -x[1]) if v))
    i_s = h.index("Warp Stall Sampling (All Samples)")
    order = sorted(range(len(data)), key=lambda j: -f(data[j][i_s]))[:ntop]
    for j in order:
        r = data[j]
        reasons = sorted(((h[i][6:], f(r[i])) for i in sc if f(r[i])), key=lambda x: -x[1])[:3]
        print(f"{f(r[i_s]) / alls * 100:5.1f}% {r[1][:60]:60s} " + " ".join(f"{a}={b / alls * 100:.1f}" for a, b in reasons))
        for k in range(max(0, j - 2), j):
            print(f"          prev: {data[k][1][:70]}")


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 20)
