"""One 2^28 u32/u32 uniform sort through the public API (for ncu captures)."""
import sys
import torch
import gen
import paper_1611_01137_b200 as hrs

n = 1 << int(sys.argv[1]) if len(sys.argv) > 1 else 1 << 28
dist = sys.argv[2] if len(sys.argv) > 2 else "uniform"
k = gen.keys(n, 32, dist, device="cuda")
v = gen.values(n, 32, "index", device="cuda")
for _ in range(2):
    ko, vo = hrs.sort(k, v)
torch.cuda.synchronize()
print("ok", bool((ko[1:].view(torch.int32).to(torch.int64) & 0xffffffff).ge((ko[:-1].view(torch.int32).to(torch.int64) & 0xffffffff)).all()))
