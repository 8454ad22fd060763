"""Summarise an `ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum
--csv` launch list: the launches of the LAST sort of the run (from its k_init), in order, with
their share of that sort's serialised time."""
import csv
import io
import sys


def main(path):
    txt = open(path).read()
    rows = list(csv.reader(io.StringIO(txt[txt.index('"ID"'):])))
    h = rows[0]
    ci = {n: h.index(n) for n in ("ID", "Kernel Name", "Metric Name", "Metric Value")}
    launches = {}
    order = []
    for r in rows[1:]:
        if len(r) < len(h):
            continue
        k = int(r[ci["ID"]])
        if k not in launches:
            launches[k] = {"name": r[ci["Kernel Name"]]}
            order.append(k)
        launches[k][r[ci["Metric Name"]]] = float(r[ci["Metric Value"]].replace(",", ""))
    inits = [k for k in order if "k_init" in launches[k]["name"]]
    last = [k for k in order if k >= inits[-1]] if inits else order
    tot = sum(launches[k].get("gpu__time_duration.sum", 0) for k in last)
    print(f"# launches of the last sort: {len(last)}; serialised total {tot / 1e3:.1f} us (ncu, cold caches)")
    agg = {}
    for k in last:
        L = launches[k]
        t = L.get("gpu__time_duration.sum", 0)
        rd, wr = L.get("dram__bytes_read.sum", 0), L.get("dram__bytes_write.sum", 0)
        print(f"{t / 1e3:9.1f} us {100 * t / tot:5.1f}%  read {rd / 1e6:9.1f} MB  write {wr / 1e6:9.1f} MB  "
              f"{L['name'][:90]}")
        base = L["name"].split("<")[0].replace("void ", "")
        a = agg.setdefault(base, [0.0, 0.0, 0.0, 0])
        a[0] += t
        a[1] += rd
        a[2] += wr
        a[3] += 1
    print("# by kernel: share of the sort, DRAM bytes")
    for base, (t, rd, wr, n) in sorted(agg.items(), key=lambda x: -x[1][0]):
        print(f"{base:20s} {n:3d} launches {100 * t / tot:5.1f}%  {t / 1e3:8.1f} us  read {rd / 1e9:.3f} GB write {wr / 1e9:.3f} GB")


if __name__ == "__main__":
    main(sys.argv[1])
