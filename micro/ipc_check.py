"""Two processes on one GPU: CUDA IPC export / open of a torch buffer and a cross-process
write through the opened address (hrs.copy_pieces with a raw destination), then the fused
distributed sort with CUDA_LAUNCH_BLOCKING for error localisation."""
import os
import socket
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402


def worker(rank, port):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=2)
    from paper_1611_01137_b200 import ipc
    buf = torch.zeros(1000, dtype=torch.int32, device="cuda:0") + rank * 100
    h = ipc.export(buf[10:])
    allh = [None, None]
    dist.all_gather_object(allh, h)
    other = ipc.open(allh[1 - rank])
    print(rank, "export", h[1:], "opened", hex(other), flush=True)
    from cuda.bindings import runtime as rt
    src = torch.arange(5, dtype=torch.int32, device="cuda:0") + 1000 * (rank + 1)
    r = rt.cudaMemcpy(other, src.data_ptr(), 20, rt.cudaMemcpyKind.cudaMemcpyDeviceToDevice)
    torch.cuda.synchronize()
    dist.barrier()
    print(rank, "memcpy rc", r[0], "buf[8:17]", buf[8:17].tolist(), flush=True)
    dist.barrier()
    import gen
    from paper_1611_01137_b200 import dist as hdist
    n = 100003
    k = gen.keys(n, 32, "uniform", start=rank * n, device="cuda:0")
    v = gen.values(n, 32, "index", start=rank * n, device="cuda:0")
    s = hdist.DistributedSorter(k, v, exchange="fused")
    try:
        ko, vo, off = s.step()
        torch.cuda.synchronize()
        print(rank, "fused ok", off, ko.numel(), flush=True)
    except Exception as e:
        print(rank, "fused failed", repr(e)[:500], flush=True)
    dist.destroy_process_group()


if __name__ == "__main__":
    with socket.socket() as sk:
        sk.bind(("127.0.0.1", 0))
        port = sk.getsockname()[1]
    mp.start_processes(worker, args=(port,), nprocs=2, start_method="spawn")
