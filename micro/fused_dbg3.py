import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, torch.distributed as dist
os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT="29533")
dist.init_process_group("gloo", rank=0, world_size=1)
import gen, oracle
from paper_1611_01137_b200 import dist as hdist
n = 70001
k = gen.keys(n, 32, "uniform", device="cuda:0")
v = gen.values(n, 32, "index", device="cuda:0")
fk, fv = oracle.sort(k.cpu(), v.cpu(), 0, 32)
for ex in ("grouped", "fused"):
    s = hdist.DistributedSorter(k, v, exchange=ex)
    for step in range(2):
        ko, vo, off = s.step()
        torch.cuda.synchronize()
        ok = np.array_equal(oracle._u64(ko.cpu()), fk), np.array_equal(oracle._u64(vo.cpu()), fv)
        print(ex, step, ok, flush=True)
        if not ok[0]:
            g = oracle._u64(ko.cpu()); bad = np.nonzero(g != fk)[0]
            print("  bad", len(bad), bad[:8], g[bad[:4]], fk[bad[:4]])
            rk = oracle._u64(s._rk[:n].cpu())
            ek, ev, eo = oracle.partition_pass(k.cpu(), v.cpu(), 24, 32)
            print("  rk == partition:", np.array_equal(rk, ek))
