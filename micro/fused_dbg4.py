import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, torch.distributed as dist
os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT="29534")
dist.init_process_group("gloo", rank=0, world_size=1)
import gen, oracle
from paper_1611_01137_b200 import dist as hdist
n = 70001
k = gen.keys(n, 32, "uniform", device="cuda:0")
v = gen.values(n, 32, "index", device="cuda:0")
s = hdist.DistributedSorter(k, v, exchange="fused")
orig = s.ops.partition_pass_to
def pp(keys, vals, lo, hi, offsets, kw, vw):
    print("called lo hi", lo, hi, "offs[:4]", offsets[:4], "kw", [hex(x) for x in kw], "rk", hex(s._rk.data_ptr()), flush=True)
    orig(keys, vals, lo, hi, offsets, kw, vw)
    torch.cuda.synchronize()
    print("rk[:4] after", s._rk[:4].tolist(), flush=True)
s.ops.partition_pass_to = pp
ko, vo, off = s.step()
torch.cuda.synchronize()
print("rk[:4] end", s._rk[:4].tolist(), "ko[:4]", ko[:4].tolist())
