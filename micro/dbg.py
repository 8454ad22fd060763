import torch, numpy as np, sys
sys.path.insert(0, '/root/repo')
import paper_1611_01137_b200 as hrs, gen, oracle
for n in (1, 2, 33, 5000):
    k = gen.keys(n, 32, 'uniform', seed=n+1)
    kd = k.cuda()
    temp = torch.empty(hrs.temp_bytes(n, 4, 0), dtype=torch.uint8, device='cuda')
    hrs.profile_enable(True)
    ko, _ = hrs.sort(kd, temp=temp)
    torch.cuda.synchronize()
    recs = hrs.profile_collect()
    st = hrs.get_stats(temp)
    ek, _ = oracle.sort(k, None, 0, 32)
    got = oracle._u64(ko.cpu())
    print(n, np.array_equal(got, ek), got[:4], ek[:4], [r[:2] for r in recs], st['local_in_class'])
    import ctypes
    ctl = temp[:512].cpu().numpy().view(np.uint32)
    print('ctl words', ctl[:80])
