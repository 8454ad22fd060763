"""One sort (twice) of a BASELINE-size workload through the public API (for ncu captures).
    python micro/prof_sort.py LOG2N KBITS DIST"""
import sys
import torch
import gen
import paper_1611_01137_b200 as hrs

n = 1 << int(sys.argv[1])
kbits = int(sys.argv[2])
dist = sys.argv[3]
k = gen.keys(n, kbits, dist, device="cuda")
v = gen.values(n, kbits, "index", device="cuda")
temp = torch.empty(hrs.temp_bytes(n, kbits // 8, kbits // 8), dtype=torch.uint8, device="cuda")
for _ in range(2):
    ko, vo = hrs.sort(k, v, temp=temp)
torch.cuda.synchronize()
st = hrs.get_stats(temp)
print({k2: st[k2] for k2 in ("counting_passes", "local_buckets", "local_recs", "merged_groups")}, st.get("local_in_class"))
