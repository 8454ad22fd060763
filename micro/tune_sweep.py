"""Sweep the local/merge thresholds (runtime tuning, no rebuild) on 2^28 records:
    python micro/tune_sweep.py KBITS DIST"""
import sys
import torch
import gen
import paper_1611_01137_b200 as hrs

kbits, dist = int(sys.argv[1]), sys.argv[2]
n = 1 << 28
k = gen.keys(n, kbits, dist, device="cuda")
v = gen.values(n, kbits, "index", device="cuda")
ko, vo = torch.empty_like(k), torch.empty_like(v)
lmax = hrs.max_local_threshold(kbits // 8, kbits // 8)
for lt in (4096, 6144, 8192):
    if lt > lmax:
        continue
    for div in (8, 4, 2, 1):
        tu = {"local_threshold": lt, "merge_threshold": max(1, lt // div)}
        temp = torch.empty(hrs.temp_bytes(n, kbits // 8, kbits // 8, tuning=tu), dtype=torch.uint8, device="cuda")
        for _ in range(2):
            hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp, tuning=tu)
        st, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        st.record()
        for _ in range(5):
            hrs.sort(k, v, keys_out=ko, values_out=vo, temp=temp, tuning=tu)
        en.record()
        torch.cuda.synchronize()
        s = hrs.get_stats(temp)
        print(f"k{kbits} {dist:8s} lt={lt} mt={tu['merge_threshold']}: {st.elapsed_time(en) / 5:.3f} ms "
              f"passes={s['counting_passes']} merged={s['merged_groups']} local_buckets={s['local_buckets']}", flush=True)
        del temp
