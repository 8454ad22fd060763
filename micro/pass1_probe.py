"""Why is the first scatter pass slower than the second on uniform 2^28 u32/u32 (c2: 1.08 vs
0.99 ms)?  Times the scatter of one pass in isolation under different layouts:
  a  c2 as is (pass 1: one bucket -> 256 sub-buckets 4 MB apart; pass 2: 256 buckets)
  b  bits [24, 32) only: pass 1 is the only pass and writes `out`
  c  top digit constant (keys & 0x00FFFFFF | 0x5A000000): pass 1 skipped (input stays), pass 2
     scatters the whole array into 256 sub-buckets 4 MB apart, reading the input
  d  bits [16, 32), top digit constant: the same spread scatter, D = 2 (writes `out`)
Run on the GPU box:  python micro/pass1_probe.py"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import gen  # noqa: E402
import paper_1611_01137_b200 as hrs  # noqa: E402


def run(tag, k, v, b0, b1):
    ko, vo = torch.empty_like(k), torch.empty_like(v)
    temp = torch.empty(hrs.temp_bytes(k.numel(), 4, 4), dtype=torch.uint8, device="cuda")
    for _ in range(3):
        hrs.sort(k, v, b0, b1, keys_out=ko, values_out=vo, temp=temp)
    torch.cuda.synchronize()
    st, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    st.record()
    for _ in range(10):
        hrs.sort(k, v, b0, b1, keys_out=ko, values_out=vo, temp=temp)
    en.record()
    torch.cuda.synchronize()
    hrs.profile_enable(True)
    for _ in range(5):
        hrs.sort(k, v, b0, b1, keys_out=ko, values_out=vo, temp=temp)
    recs = hrs.profile_collect()
    hrs.profile_enable(False)
    per = {}
    for kind, p, ms in recs:
        per.setdefault(f"{kind}{p}", []).append(ms)
    print(f"{tag:3s} bits [{b0},{b1}) step={st.elapsed_time(en) / 10:.3f} ms " + " ".join(
        f"{a}={sum(x) / len(x):.3f}" for a, x in sorted(per.items()) if sum(x) / len(x) > 0.02), flush=True)


def main():
    n = 1 << 28
    k = gen.keys(n, 32, "uniform", device="cuda")
    v = gen.values(n, 32, "index", device="cuda")
    run("a", k, v, 0, 32)
    run("b", k, v, 24, 32)
    kc = (k.view(torch.int32) & 0x00FFFFFF | 0x5A000000).view(torch.uint32)
    run("c", kc, v, 0, 32)
    run("d", kc, v, 16, 32)
    run("b2", k, v, 16, 32)


if __name__ == "__main__":
    main()
