"""c1 latency of a libhrs variant: python micro/c1_exp.py NAME [log2n] [kbits] [vbits]"""
import os
import sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
os.environ["HRS_LIB"] = os.path.join(ROOT, "micro", f"libhrs_{sys.argv[1]}.so")
sys.path.insert(0, ROOT)
import torch  # noqa: E402
import gen  # noqa: E402
import paper_1611_01137_b200 as hrs  # noqa: E402
logn = int(sys.argv[2]) if len(sys.argv) > 2 else 20
kbits = int(sys.argv[3]) if len(sys.argv) > 3 else 32
vbits = int(sys.argv[4]) if len(sys.argv) > 4 else 0
n = 1 << logn
k = gen.keys(n, kbits, "uniform", device="cuda")
v = gen.values(n, vbits, "index", device="cuda") if vbits else None
ko = torch.empty_like(k)
vo = torch.empty_like(v) if vbits else None
temp = torch.empty(hrs.temp_bytes(n, kbits // 8, vbits // 8), dtype=torch.uint8, device="cuda")
for _ in range(5):
    hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp)
st, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
st.record()
R = 50
for _ in range(R):
    hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp)
en.record()
torch.cuda.synchronize()
print(f"{sys.argv[1]:8s} 2^{logn} k{kbits}v{vbits}: {st.elapsed_time(en) / R * 1000:.1f} us/sort")
