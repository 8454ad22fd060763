import os, socket, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch, torch.distributed as dist, torch.multiprocessing as mp


def worker(rank, port, world):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    import gen
    from paper_1611_01137_b200 import dist as hdist
    n = 100003
    k = gen.keys(n, 32, "uniform", start=rank * n, device="cuda:0")
    v = gen.values(n, 32, "index", start=rank * n, device="cuda:0")
    s = hdist.DistributedSorter(k, v, exchange="fused")
    orig = s.ops.partition_pass_to
    def pp(keys, vals, lo, hi, offsets, kw, vw):
        print(rank, "windows", [hex(x) for x in kw], [hex(x) for x in vw], "rk", hex(s._rk.data_ptr()), s._rk.numel(),
              "kp", hex(s._kp.data_ptr()), flush=True)
        print(rank, "offs", [(o >> 48, o & ((1 << 48) - 1)) for o in offsets[:6]], "...", [(o >> 48, o & ((1 << 48) - 1)) for o in offsets[-3:]], flush=True)
        orig(keys, vals, lo, hi, offsets, kw, vw)
        torch.cuda.synchronize()
        print(rank, "pass ok", flush=True)
    s.ops.partition_pass_to = pp
    try:
        ko, vo, off = s.step()
        torch.cuda.synchronize()
        print(rank, "fused ok", off, ko.numel(), flush=True)
    except Exception as e:
        print(rank, "fused failed", repr(e)[:300], flush=True)
    dist.destroy_process_group()


if __name__ == "__main__":
    world = int(sys.argv[1])
    with socket.socket() as sk:
        sk.bind(("127.0.0.1", 0))
        port = sk.getsockname()[1]
    mp.start_processes(worker, args=(port, world), nprocs=world, start_method="spawn")
