"""Time libhrs variants built with different compile-time defines on 2^28 u32/u32 pairs.
Builds are made on the CPU box:  python micro/scatter_exp.py build NAME "DEF=1 DEF2=3" ...
then on the GPU box:             python micro/scatter_exp.py run NAME [dist]"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def build(name, defs):
    import importlib.util
    spec = importlib.util.spec_from_file_location("b", os.path.join(ROOT, "paper_1611_01137_b200", "build.py"))
    b = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(b)
    b.build(force=True, out=os.path.join(ROOT, "micro", f"libhrs_{name}.so"), defines=defs.split())


def run(name, dist="uniform", kbits=32):
    os.environ["HRS_LIB"] = os.path.join(ROOT, "micro", f"libhrs_{name}.so")
    sys.path.insert(0, ROOT)
    import torch
    import gen
    import paper_1611_01137_b200 as hrs
    n = 1 << 28
    kbits = int(kbits)
    k = gen.keys(n, kbits, dist, device="cuda")
    val = gen.values(n, kbits, "index", device="cuda")
    ko, vo = torch.empty_like(k), torch.empty_like(val)
    temp = torch.empty(hrs.temp_bytes(n, kbits // 8, kbits // 8), dtype=torch.uint8, device="cuda")
    for _ in range(3):
        hrs.sort(k, val, keys_out=ko, values_out=vo, temp=temp)
    st, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    st.record()
    for _ in range(10):
        hrs.sort(k, val, keys_out=ko, values_out=vo, temp=temp)
    en.record()
    torch.cuda.synchronize()
    tot = st.elapsed_time(en) / 10
    hrs.profile_enable(True)
    for _ in range(5):
        hrs.sort(k, val, keys_out=ko, values_out=vo, temp=temp)
    recs = hrs.profile_collect()
    per = {}
    for kind, p, ms in recs:
        per.setdefault(f"{kind}{p}", []).append(ms)
    if kbits == 32:
        k64 = k.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
        sk, si = torch.sort(k64, stable=True)
        ok = bool(torch.equal(ko.view(torch.int32).to(torch.int64) & 0xFFFFFFFF, sk)) and \
            bool(torch.equal(vo.view(torch.int32).to(torch.int64), si))
    else:  # O(n) certificate: values = index, keys_out[i] = keys[values_out[i]], (key, value) increasing
        kk, vv = ko.view(torch.int64), vo.view(torch.int64)
        ok = bool(torch.equal(k.view(torch.int64)[vv], kk))
        a, b = kk[:-1] ^ (-(2 ** 63)), kk[1:] ^ (-(2 ** 63))  # unsigned order as signed
        ok = ok and bool(((a < b) | ((a == b) & (vv[:-1] < vv[1:]))).all())
    print(f"{name:12s} {dist:8s} k{kbits} {'OK ' if ok else 'BAD'} step={tot:.3f} ms " + " ".join(
        f"{k2}={sum(x) / len(x):.3f}" for k2, x in sorted(per.items()) if sum(x) / len(x) > 0.009), flush=True)


if __name__ == "__main__":
    if sys.argv[1] == "build":
        for i in range(2, len(sys.argv), 2):
            build(sys.argv[i], sys.argv[i + 1])
    else:
        run(sys.argv[2], *(sys.argv[3:5]))
