"""Summarise an `ncu --page source --csv --print-source sass` export: top stall lines and opcode mix."""
import csv
import sys
from collections import Counter


def main(path, ntop=25):
    rows = list(csv.reader(open(path)))
    hdr_i = next(i for i, r in enumerate(rows) if "Source" in r and "Address" in r)
    hdr = rows[hdr_i]
    data = [r for r in rows[hdr_i + 1:] if len(r) == len(hdr)]

    def f(x):
        try:
            return float(x)
        except ValueError:
            return 0.0
    i_src, i_s, i_e = hdr.index("Source"), hdr.index("Warp Stall Sampling (All Samples)"), hdr.index("Instructions Executed")
    tot = sum(f(r[i_s]) for r in data) or 1
    for r in sorted(data, key=lambda r: -f(r[i_s]))[:ntop]:
        print(f"{f(r[i_s]) / tot * 100:5.1f}%  exec={int(f(r[i_e])):>10}  {r[hdr.index('Address')]} {r[i_src][:100]}")
    c = Counter()
    for r in data:
        toks = r[i_src].split()
        if not toks:
            continue
        op = toks[1] if toks[0].startswith("@") and len(toks) > 1 else toks[0]
        c[op.split(".")[0]] += int(f(r[i_e]))
    total = sum(c.values())
    print("opcode mix (warp instructions executed):", total)
    for op, n in c.most_common(25):
        print(f"  {op:10s} {n:>12d} {n / total * 100:5.1f}%")


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 25)
