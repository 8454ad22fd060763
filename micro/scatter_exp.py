"""Time k_scatter variants (HRS_EXP compile flag) on 2^28 u32/u32 uniform pairs.
Builds are made on the CPU box: python micro/scatter_exp.py build; run on the GPU box."""
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
VARIANTS = {0: "product", 1: "no global stores", 3: "contiguous stores (no scatter)",
            10: "local: balanced kpt", 11: "local: 2 chains/warp", 12: "local: balanced + 2 chains",
            }


def build():
    import importlib.util
    spec = importlib.util.spec_from_file_location("b", os.path.join(ROOT, "paper_1611_01137_b200", "build.py"))
    b = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(b)
    for v in (sys.argv[2:] and map(int, sys.argv[2:])) or VARIANTS:
        b.build(force=True, out=os.path.join(ROOT, "micro", f"libhrs_exp{v}.so"), defines=[f"HRS_EXP={v}"])


def run(v):
    os.environ["HRS_LIB"] = os.path.join(ROOT, "micro", f"libhrs_exp{v}.so")
    sys.path.insert(0, ROOT)
    import torch
    import gen
    import paper_1611_01137_b200 as hrs
    n = 1 << 28
    k = gen.keys(n, 32, sys.argv[3] if len(sys.argv) > 3 else "uniform", device="cuda")
    val = gen.values(n, 32, "index", device="cuda")
    ko, vo = torch.empty_like(k), torch.empty_like(val)
    temp = torch.empty(hrs.temp_bytes(n, 4, 4), dtype=torch.uint8, device="cuda")
    for _ in range(3):
        hrs.sort(k, val, keys_out=ko, values_out=vo, temp=temp)
    hrs.profile_enable(True)
    for _ in range(5):
        hrs.sort(k, val, keys_out=ko, values_out=vo, temp=temp)
    recs = hrs.profile_collect()
    per = {}
    for kind, p, ms in recs:
        per.setdefault(f"{kind}{p}", []).append(ms)
    k64 = k.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    sk, si = torch.sort(k64, stable=True)
    ok = bool(torch.equal(ko.view(torch.int32).to(torch.int64) & 0xFFFFFFFF, sk)) and \
        bool(torch.equal(vo.view(torch.int32).to(torch.int64), si))
    print(f"exp{v} {'OK ' if ok else 'BAD'} {VARIANTS[v]:32s} " + " ".join(f"{k2}={sum(x)/len(x):.3f}" for k2, x in sorted(per.items())
                                                 if sum(x) / len(x) > 0.02))


if __name__ == "__main__":
    if sys.argv[1] == "build":
        build()
    else:
        run(int(sys.argv[2]))
