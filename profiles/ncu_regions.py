"""Split a kernel's SASS (from `ncu --page source --csv --print-source sass`) into the
regions between block barriers: executed warp instructions, stall samples (and the top
reasons) and shared-memory wavefronts per region -- where a barrier-phased kernel spends
its issue slots and its time."""
import csv
import gzip
import sys


def main(path):
    op = gzip.open if path.endswith(".gz") else open
    rows = list(csv.reader(op(path, "rt", errors="replace")))
    hi = next(i for i, r in enumerate(rows) if "Source" in r and "Address" in r)
    h = rows[hi]
    data, seen = [], set()
    for r in rows[hi + 1:]:
        if len(r) == len(h) and r[0].startswith("0x") and r[0] not in seen:
            seen.add(r[0])
            data.append(r)
    f = lambda x: float(x) if x not in ("", None) else 0.0
    ix, iss, iwf = h.index("Instructions Executed"), h.index("Warp Stall Sampling (All Samples)"), h.index("L1 Wavefronts Shared")
    sc = [i for i, n in enumerate(h) if n.startswith("stall_")]
    tot_i = sum(f(r[ix]) for r in data) or 1
    tot_s = sum(f(r[iss]) for r in data) or 1
    tot_w = sum(f(r[iwf]) for r in data) or 1
    reg, regs = None, []
    for k, r in enumerate(data):
        if reg is None or "BAR.SYNC" in r[1]:
            reg = {"start": k, "first": r[1].strip()[:40], "inst": 0.0, "samp": 0.0, "wf": 0.0, "st": {}, "n": 0}
            regs.append(reg)
        reg["inst"] += f(r[ix])
        reg["samp"] += f(r[iss])
        reg["wf"] += f(r[iwf])
        reg["n"] += 1
        for i in sc:
            reg["st"][h[i][6:]] = reg["st"].get(h[i][6:], 0.0) + f(r[i])
    print(f"total: {tot_i:.4g} warp inst, {tot_s:.4g} stall samples, {tot_w:.4g} smem wavefronts")
    print(" sass#  nsass   inst%  samp%   wf%   top stalls (% of all samples)")
    for g in regs:
        if g["inst"] / tot_i < 0.002 and g["samp"] / tot_s < 0.002:
            continue
        top = sorted(g["st"].items(), key=lambda x: -x[1])[:4]
        print(f"{g['start']:6d} {g['n']:6d} {g['inst'] / tot_i * 100:6.1f} {g['samp'] / tot_s * 100:6.1f} {g['wf'] / tot_w * 100:5.1f}   "
              + " ".join(f"{a}={b / tot_s * 100:.1f}" for a, b in top if b) + f"   [{g['first']}]")


if __name__ == "__main__":
    main(sys.argv[1])
