"""torchrun --nproc-per-node N micro/dist_nccl_check.py: the distributed driver over NCCL
(device tensors, no host staging) on 2^24 records per rank, checked with the O(n)
certificate on each rank's slice and the rank boundaries."""
import os
import sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402
import gen  # noqa: E402
from paper_1611_01137_b200 import dist as hdist  # noqa: E402

rank, world = int(os.environ.get("RANK", 0)), int(os.environ.get("WORLD_SIZE", 1))
dev = torch.device("cuda", int(os.environ.get("LOCAL_RANK", 0)))
torch.cuda.set_device(dev)
dist.init_process_group("nccl", device_id=dev)
n = 1 << 24
for d in ("uniform", "and3"):
    k = gen.keys(n, 32, d, start=rank * n, device=dev)
    v = gen.values(n, 32, "index", start=rank * n, device=dev)
    ko, vo, off = hdist.DistributedSorter(k, v).step()
    torch.cuda.synchronize()
    idx = vo.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    full = gen.keys(n * world, 32, d, device=dev).view(torch.int32)
    ok = torch.equal(full[idx], ko.view(torch.int32))
    sk = ko.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    ok = ok and bool(((sk[:-1] < sk[1:]) | ((sk[:-1] == sk[1:]) & (idx[:-1] < idx[1:]))).all())
    print(f"rank {rank}/{world} {d}: n_out={ko.numel()} offset={off} certificate={'OK' if ok else 'BAD'}", flush=True)
dist.destroy_process_group()
