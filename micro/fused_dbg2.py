import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import gen, oracle
import paper_1611_01137_b200 as hrs
n = 70001
k = gen.keys(n, 32, "uniform", device="cuda:0")
v = gen.values(n, 32, "index", device="cuda:0")
h = hrs.digit_histogram(k, 24, 32).view(torch.int64).cpu().numpy()
C = np.concatenate([[0], np.cumsum(h)])
rk = torch.zeros(n, dtype=torch.uint32, device="cuda:0"); rv = torch.zeros_like(rk)
kp = torch.zeros_like(rk); vp = torch.zeros_like(rk)
offs = [int(C[b]) for b in range(256)]
hrs.partition_pass_to(k, v, 24, 32, offs, [rk.data_ptr(), kp.data_ptr()], [rv.data_ptr(), vp.data_ptr()])
torch.cuda.synchronize()
ek, ev, eo = oracle.partition_pass(k.cpu(), v.cpu(), 24, 32)
gk = oracle._u64(rk.cpu()); gv = oracle._u64(rv.cpu())
print("partition keys equal", np.array_equal(gk, ek), "values", np.array_equal(gv, ev), "offs equal", np.array_equal(eo[:-1], C[:-1]))
bad = np.nonzero(gk != ek)[0]
print("first bad", bad[:10], gk[bad[:5]] if len(bad) else None, ek[bad[:5]] if len(bad) else None)
ko, vo = hrs.sort_grouped(rk, rv, h.tolist())
torch.cuda.synchronize()
fk, fv = oracle.sort(k.cpu(), v.cpu(), 0, 32)
print("sorted equal", np.array_equal(oracle._u64(ko.cpu()), fk), np.array_equal(oracle._u64(vo.cpu()), fv))
