#!/usr/bin/env python
"""Benchmark of the stable hybrid MSD radix sort on B200 (one JSON line on rank 0).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config c2] [--dist uniform]
    python bench.py --impl reference ...      # the CPU oracle on a bounded sample

Metric (BASELINE.json): sorted records/s and the fraction of the HBM roofline.  A
"step" is one full sort (every counting pass, the classification and every local
sort) of the configured synthetic workload, inputs resident in HBM.  Default config
c2 = 2^28 uint32 keys + uint32 values, uniform (BASELINE.json configs[1]); the
inputs (2 GiB + outputs + aux) are far larger than the 126 MB L2, so no flush is
needed between steps.

Multi-GPU (torchrun, N > 1): every rank sorts its own 2^28-record shard of a global
N * 2^28 input through the distributed driver (first-digit histogram all-gather,
bucket assignment, stable partition, NCCL all-to-all, local sort); value = N * 2^28
records / max-over-ranks step time ("weak" scaling).
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

CONFIGS = {
    # name: (log2 n, key bits, value bits, description)
    "c1": (20, 32, 0, "2^20 uniform uint32 keys, keys-only"),
    "c2": (28, 32, 32, "2^28 uint32 key + uint32 value pairs"),
    "c3": (28, 32, 32, "2^28 uint32 key + uint32 value pairs, AND-skewed"),
    "c4": (28, 64, 64, "2^28 uint64 key + uint64 value pairs"),
    # BASELINE.json configs[4]: 64 GiB of u64/u64 records in total, split over the N GPUs
    # (strong scaling); needs N >= 2 (input + output + aux of 64 GiB exceed one GPU's HBM)
    "c5": (32, 64, 64, "2^32 uint64 key + uint64 value pairs (64 GiB) in total"),
}
STRONG = {"c5"}
METRIC = "sorted records/sec and % of B200 HBM roofline (1/2/4/8 GPU)"


def _peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            p = json.load(f)
        return float(p["hbm_gbs"]), "measured"
    except Exception:
        return 6650.0, "fallback"


class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled during the timed region."""

    FIELDS = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,"
              "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
              "clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index = index
        self.samples = []
        self.proc = None
        self.thread = None

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "100"], stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except Exception:
            self.proc = None
            return
        self.thread = threading.Thread(target=self._read, daemon=True)
        self.thread.start()

    def _read(self):
        for line in self.proc.stdout:
            parts = [x.strip() for x in line.split(",")]
            if len(parts) == 6:
                self.samples.append(parts)

    def stop(self) -> dict:
        if self.proc is None:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        time.sleep(0.25)
        self.proc.terminate()
        try:
            self.proc.wait(timeout=2)
        except Exception:
            self.proc.kill()
        sm = [float(s[0]) for s in self.samples if s[0].replace(".", "").isdigit()]
        mx = [float(s[1]) for s in self.samples if s[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for s in self.samples for i in range(4) if s[2 + i].lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.samples)}


def _env_rank():
    return int(os.environ.get("RANK", "0")), int(os.environ.get("WORLD_SIZE", "1")), \
        int(os.environ.get("LOCAL_RANK", "0"))


# ---------------------------------------------------------------------------- reference arm

def run_reference(args):
    """The CPU oracle (oracle/oracle.c, single-threaded LSD) as it stands, one bounded
    sample of the configured workload per step."""
    rank, world, _ = _env_rank()
    if rank != 0:
        return 0
    import numpy as np
    import gen
    import oracle
    logn, kbits, vbits, desc = CONFIGS[args.config]
    n = min(1 << logn, 1 << args.ref_log2)
    k = oracle._u64(gen.keys(n, kbits, args.dist))
    v = np.arange(n, dtype=np.uint64) if vbits else None
    for _ in range(args.warmup):
        oracle.sort(k, v, 0, kbits)
    times = []
    for _ in range(args.steps):
        t0 = time.perf_counter()
        oracle.sort(k, v, 0, kbits)
        times.append(time.perf_counter() - t0)
    t = sum(times) / len(times)
    value = n / t
    unit = "records/s"
    sample = f"{n} records ({args.dist}) of the {desc} workload per step, single-threaded LSD oracle"
    line = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": unit, "n_gpus": world,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": t * 1e3, "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "u32" if kbits == 32 else "u64", "data": "synthetic",
        "config": {"workload": f"{args.config}:{desc}, {args.dist}", "n": n, "key_bits": kbits,
                   "value_bits": vbits, "parallelism": f"cpu1"},
        "cpu_baseline": {"value": value, "unit": unit, "cores": 1, "kind": "oracle", "sample": sample},
        "e2e": {"value": value, "unit": unit, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


# ---------------------------------------------------------------------------- product arm

def _events(torch, k):
    return [torch.cuda.Event(enable_timing=True) for _ in range(k)]


def run_hrs(args):
    import torch

    import gen
    import paper_1611_01137_b200 as hrs

    rank, world, local_rank = _env_rank()
    torch.cuda.set_device(local_rank)
    dev = torch.device("cuda", local_rank)
    logn, kbits, vbits, desc = CONFIGS[args.config]
    dist_name = args.dist
    if args.config == "c3" and dist_name == "uniform":
        dist_name = "and3"
    strong = args.config in STRONG
    n = (1 << logn) // world if strong else 1 << logn  # records per GPU
    if strong and world < 2 and not args.force_dist:
        if rank == 0:
            print(json.dumps({"metric": METRIC, "config": {"workload": f"{args.config}:{desc}"}, "n_gpus": world,
                              "unavailable": "64 GiB of input plus its output and aux exceed one GPU's HBM; "
                                             "c5 runs at N >= 2 (or one rank's shard with --force-dist)"}))
        return 0
    kb, vb = kbits // 8, vbits // 8
    pg = None
    use_dist = world > 1 or args.force_dist
    if use_dist:
        import torch.distributed as dist
        if "RANK" not in os.environ:  # --force-dist without torchrun: a world of one
            import socket
            with socket.socket() as sk:
                sk.bind(("127.0.0.1", 0))
                os.environ.setdefault("MASTER_PORT", str(sk.getsockname()[1]))
            os.environ.update(RANK="0", WORLD_SIZE="1", LOCAL_RANK="0")
            os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
        import datetime
        # a hung collective (a dead peer) fails the run after this long instead of blocking it
        dist.init_process_group("nccl", device_id=dev, timeout=datetime.timedelta(seconds=args.nccl_timeout))
        pg = dist.group.WORLD

    seed = gen.SEEDS[0]
    keys = gen.keys(n, kbits, dist_name, seed=seed, start=rank * n, device=dev)
    vals = gen.values(n, vbits, "index", start=rank * n, device=dev) if vbits else None
    stream = torch.cuda.current_stream()

    if use_dist:
        from paper_1611_01137_b200 import dist as hdist
        sorter = hdist.DistributedSorter(keys, vals, group=pg, exchange=args.exchange)
        step = sorter.step
    else:
        keys_out = torch.empty_like(keys)
        vals_out = torch.empty_like(vals) if vals is not None else None
        temp = torch.empty(hrs.temp_bytes(n, kb, vb), dtype=torch.uint8, device=dev)

        def step():
            hrs.sort(keys, vals, keys_out=keys_out, values_out=vals_out, temp=temp)

    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()

    # ---------------- timed region: K steps, barrier + synchronize on both sides
    sampler = ClockSampler(local_rank)
    sampler.start()
    time.sleep(0.3)
    if pg is not None:
        torch.distributed.barrier()
    torch.cuda.synchronize()
    l0 = hrs.launch_count()
    ev = _events(torch, args.steps + 1)
    ev[0].record(stream)
    for i in range(args.steps):
        step()
        ev[i + 1].record(stream)
    torch.cuda.synchronize()
    launches = hrs.launch_count() - l0
    if pg is not None:
        torch.distributed.barrier()
    clocks = sampler.stop()
    step_ms = [ev[i].elapsed_time(ev[i + 1]) for i in range(args.steps)]
    t_ms = sum(step_ms) / len(step_ms)
    if pg is not None:
        tt = torch.tensor([t_ms], dtype=torch.float64, device=dev)
        torch.distributed.all_reduce(tt, op=torch.distributed.ReduceOp.MAX)
        t_ms = float(tt.item())
    total = n * world
    value = total / (t_ms * 1e-3)

    peak, peak_kind = _peaks()
    out = {"metric": METRIC, "value": value, "unit": "records/s", "n_gpus": world, "steps": args.steps,
           "warmup": args.warmup, "ms_per_step": t_ms, "higher_is_better": True,
           "scaling": "strong" if strong else "weak",
           "vs_baseline": None, "dtype": "u32" if kbits == 32 else "u64", "data": "synthetic",
           "config": {"workload": f"{args.config}:{desc}, {dist_name}", "n_per_gpu": n, "key_bits": kbits,
                      "value_bits": vbits, "bits": [0, kbits], "values": "input index",
                      "parallelism": f"dp{world}" if world > 1 else "single",
                      "exchange": args.exchange if use_dist else None,
                      "l2": "inputs (>= 2 GiB) larger than the 126 MB L2; no flush"},
           "gpu_launches": launches, "clocks": clocks,
           "step_ms": {"median": statistics.median(step_ms), "min": min(step_ms), "max": max(step_ms)}}

    if use_dist:
        out["exchange"] = run_exchange(torch, sorter, pg, dev, kb, vb)
        if not args.no_e2e:
            out["e2e"] = run_e2e_dist(torch, sorter, pg, args, n, dev)
    else:
        st = hrs.get_stats(temp)
        bmin = st["bytes_min"]
        out["sort_roofline"] = {
            "bytes_min": bmin, "bytes_per_record": bmin / n, "peak_gbs": peak, "peak": peak_kind,
            "achieved_gbs": bmin / (t_ms * 1e-3) / 1e9, "frac": bmin / (t_ms * 1e-3) / (peak * 1e9),
            "frac_of_8tbs": bmin / (t_ms * 1e-3) / 8.0e12, "sort_rate_GBps": n * (kb + vb) / (t_ms * 1e-3) / 1e9,
            "counting_passes": st["counting_passes"], "recs_in_pass": st["recs_in_pass"],
            "local_recs": st["local_recs"], "local_buckets": st["local_buckets"],
            "merged_groups": st["merged_groups"]}
        # ---------------- per-kernel breakdown: the same K steps again, each launch bracketed by events
        hrs.profile_enable(True)
        for _ in range(args.steps):
            step()
        recs = hrs.profile_collect()
        hrs.profile_enable(False)
        per = {}
        for kind, p, ms in recs:
            key = f"{kind}{p}" if kind in ("hist", "scatter", "local", "classify") else kind
            per.setdefault(key, []).append(ms)
        kern = {k2: sum(v2) / args.steps for k2, v2 in per.items()}
        out["kernels_ms_per_step"] = {k2: round(v2, 4) for k2, v2 in sorted(kern.items())}
        # dominant kernel: the scatter (2(K+V) bytes per record it moves: the records of every
        # counting pass minus those of skipped buckets, reading #22)
        skipped = st.get("skipped_recs_in_pass", [0] * len(st["recs_in_pass"]))
        sc_bytes = sum((r - sk) * 2 * (kb + vb) for r, sk in zip(st["recs_in_pass"], skipped))
        sc_ms = sum(v2 for k2, v2 in kern.items() if k2.startswith("scatter"))
        traffic = None
        tpath = os.path.join(ROOT, "profiles", "traffic.json")
        if os.path.exists(tpath):
            try:
                tj = json.load(open(tpath))
                traffic = tj.get(f"{args.config}:{dist_name}", {}).get("scatter_dram_bytes_per_step")
            except Exception:
                traffic = None
        if sc_ms > 0:
            ach = sc_bytes / (sc_ms * 1e-3) / 1e9
            out["roofline"] = {"bound": "hbm", "kernel": "k_scatter (all counting passes)", "achieved": ach,
                               "peak": peak, "unit": "GB/s", "frac": ach / peak, "traffic": traffic,
                               "algorithmic_bytes": sc_bytes, "share_of_step": sc_ms / sum(kern.values()),
                               "peak_source": peak_kind}
        # ---------------- end to end through the public API with host buffers
        if not args.no_e2e:
            out["e2e"] = run_e2e(torch, hrs, keys, vals, temp, args, n, kb, vb)
        # ---------------- CPU baseline: the oracle as it stands on a bounded sample
        if not args.no_cpu:
            out["cpu_baseline"] = cpu_baseline(args, kbits, vbits, dist_name, keys_dev=keys)
    if rank == 0:
        print(json.dumps(out), flush=True)
    if pg is not None:
        torch.distributed.destroy_process_group()
    return 0


def _max_over_ranks(torch, x, pg, dev):
    if pg is None:
        return x
    t = torch.tensor([x], dtype=torch.float64, device=dev)
    torch.distributed.all_reduce(t, op=torch.distributed.ReduceOp.MAX, group=pg)
    return float(t.item())


def run_exchange(torch, sorter, pg, dev, kb, vb, reps=3):
    """The NCCL all-to-all of the distributed sort (step 4) against NVLink: bytes this
    rank sends to other ranks / the exchange's CUDA-event time, max time over ranks."""
    sorter.time_exchange = True
    ms = []
    for _ in range(reps):
        sorter.step()
        torch.cuda.synchronize()
        e0, e1 = sorter.exchange_events
        ms.append(e0.elapsed_time(e1))
    sorter.time_exchange = False
    me = sorter.rank
    sent = sum(c for j, c in enumerate(sorter.last["send"]) if j != me) * (kb + vb)
    recv = sum(c for j, c in enumerate(sorter.last["recv"]) if j != me) * (kb + vb)
    t = _max_over_ranks(torch, statistics.median(ms), pg, dev)
    peak = 900.0  # NVLink 5 per direction per GPU (GB/s), nominal
    ach = sent / (t * 1e-3) / 1e9 if t > 0 else 0.0
    return {"bound": "nvlink", "ms": t, "bytes_sent_to_peers": sent, "bytes_recv_from_peers": recv,
            "achieved": ach, "peak": peak, "unit": "GB/s", "frac": ach / peak, "peak_source": "nominal",
            "imbalance": sorter.last.get("imbalance"), "refine_levels": sorter.last.get("refine_levels"),
            "note": "rank 0's peer bytes over the max-over-ranks all-to-all time (keys + values)"}


def run_e2e_dist(torch, sorter, pg, args, n, dev):
    """End to end at N GPUs: every step copies this rank's shard H2D from pinned memory
    into the sorter's input tensors, runs the distributed sort (hrs.dist), and copies
    this rank's sorted slice D2H; CUDA events on the current stream, max over ranks."""
    hk = torch.empty(sorter.keys.shape, dtype=sorter.keys.dtype, pin_memory=True)
    hk.copy_(sorter.keys)
    hv = None
    if sorter.vals is not None:
        hv = torch.empty(sorter.vals.shape, dtype=sorter.vals.dtype, pin_memory=True)
        hv.copy_(sorter.vals)
    hko = torch.empty(2 * n, dtype=sorter.keys.dtype, pin_memory=True)
    hvo = torch.empty(2 * n, dtype=sorter.vals.dtype, pin_memory=True) if hv is not None else None
    k = max(4, args.steps)
    stream = torch.cuda.current_stream()

    def step():
        sorter.keys.copy_(hk, non_blocking=True)
        if hv is not None:
            sorter.vals.copy_(hv, non_blocking=True)
        ko, vo, _ = sorter.step()
        hko[:ko.numel()].copy_(ko, non_blocking=True)
        if vo is not None:
            hvo[:vo.numel()].copy_(vo, non_blocking=True)
        return ko.numel()

    step()
    torch.cuda.synchronize()
    if pg is not None:
        torch.distributed.barrier(group=pg)
    t0, t1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    t0.record(stream)
    got = 0
    for _ in range(k):
        got = step()
    t1.record(stream)
    torch.cuda.synchronize()
    t = _max_over_ranks(torch, t0.elapsed_time(t1) / k, pg, dev)
    world = sorter.world
    nb_in = n * (sorter.keys.element_size() + (sorter.vals.element_size() if hv is not None else 0))
    nb_out = got * (sorter.keys.element_size() + (sorter.vals.element_size() if hv is not None else 0))
    return {"value": n * world / (t * 1e-3), "unit": "records/s", "ms_per_step": t, "h2d_bytes_per_step": nb_in,
            "d2h_bytes_per_step": nb_out, "steps": k,
            "path": "pinned host -> H2D -> hrs.dist (partition, NCCL all-to-all, C-ABI local sort) -> D2H, per rank"}


def run_e2e(torch, hrs, keys, vals, temp, args, n, kb, vb):
    """Through the public API from pinned host memory and back, every step: H2D of the
    step's keys (+ values), hrs.sort, D2H of the sorted keys (+ values).  Consecutive
    steps are pipelined over three streams with two device buffer sets, so step i+1's
    H2D (host -> device direction) overlaps step i's sort and D2H (device -> host); each
    step still moves all of its bytes both ways inside the timed region."""
    hk = torch.empty(keys.shape, dtype=keys.dtype, pin_memory=True)
    hk.copy_(keys)
    hv = None
    if vals is not None:
        hv = torch.empty(vals.shape, dtype=vals.dtype, pin_memory=True)
        hv.copy_(vals)
    hko = torch.empty_like(hk, pin_memory=True)
    hvo = torch.empty_like(hv, pin_memory=True) if hv is not None else None
    sets = []
    for i in range(2):
        sets.append({"dk": torch.empty_like(keys), "dko": torch.empty_like(keys),
                     "dv": torch.empty_like(vals) if vals is not None else None,
                     "dvo": torch.empty_like(vals) if vals is not None else None,
                     "temp": temp if i == 0 else torch.empty_like(temp)})
    s_in, s_sort, s_out = torch.cuda.Stream(), torch.cuda.Stream(), torch.cuda.Stream()
    for b in sets:
        b["sorted"] = torch.cuda.Event()
        b["drained"] = torch.cuda.Event()
        b["loaded"] = torch.cuda.Event()
        b["sorted"].record(s_sort)
        b["drained"].record(s_out)

    def step(i):
        b = sets[i % 2]
        s_in.wait_event(b["sorted"])            # the set's inputs were consumed by its last sort
        with torch.cuda.stream(s_in):
            b["dk"].copy_(hk, non_blocking=True)
            if hv is not None:
                b["dv"].copy_(hv, non_blocking=True)
        b["loaded"].record(s_in)
        s_sort.wait_event(b["loaded"])
        s_sort.wait_event(b["drained"])         # its outputs were read back
        hrs.sort(b["dk"], b["dv"], keys_out=b["dko"], values_out=b["dvo"], temp=b["temp"], stream=s_sort)
        b["sorted"].record(s_sort)
        s_out.wait_event(b["sorted"])
        with torch.cuda.stream(s_out):
            hko.copy_(b["dko"], non_blocking=True)
            if hvo is not None:
                hvo.copy_(b["dvo"], non_blocking=True)
        b["drained"].record(s_out)

    for i in range(2):
        step(i)
    torch.cuda.synchronize()
    k = max(4, args.steps)  # the same K as the device-timed steps (at least 4)
    t0, t1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    t0.record(s_in)
    s_out.wait_event(t0)
    for i in range(k):
        step(i)
    t1.record(s_out)
    torch.cuda.synchronize()
    t = t0.elapsed_time(t1) / k
    nb = n * (kb + vb)
    return {"value": n / (t * 1e-3), "unit": "records/s", "ms_per_step": t, "h2d_bytes_per_step": nb,
            "d2h_bytes_per_step": nb, "steps": k,
            "path": "pinned host -> H2D -> hrs.sort (C ABI) -> D2H, consecutive steps pipelined over 3 streams"}


def cpu_baseline(args, kbits, vbits, dist_name, keys_dev=None):
    """The CPU baselines of SURVEY §8(d) on this box's host, bounded to ~10-30 s:
      * value: the stable LSD radix sort over every core this process may use
        (oracle/cpu_baseline.cc, byte-identical to the oracle; pinned by tests/test_oracle.py)
        on the FULL workload (the GPU input copied to the host, untimed);
      * oracle_1core: the oracle as it stands (oracle/oracle.c, one thread) on a 2^cpu_log2 slice;
      * stable_sort_1core: std::stable_sort of the records on the same slice."""
    import numpy as np
    import gen
    import oracle
    n_full = None
    if keys_dev is not None:
        k = oracle._native(keys_dev.cpu())
        n_full = k.size
    else:
        k = oracle._native(gen.keys(1 << args.cpu_log2, kbits, dist_name))
    vdt = np.uint32 if vbits == 32 else np.uint64
    v = np.arange(k.size, dtype=vdt) if vbits else None
    cores = oracle.host_cores()
    oracle.cpu_lsd_sort(k[:1 << 16], None if v is None else v[:1 << 16], 0, kbits, threads=cores)  # warm
    t0 = time.perf_counter()
    oracle.cpu_lsd_sort(k, v, 0, kbits, threads=cores)
    t_par = time.perf_counter() - t0
    ns = min(k.size, 1 << args.cpu_log2)
    ks = k[:ns].copy()
    vs = None if v is None else v[:ns].copy()
    t0 = time.perf_counter()
    oracle.sort(ks, vs, 0, kbits)
    t_or = time.perf_counter() - t0
    t0 = time.perf_counter()
    oracle.cpu_stable_sort(ks, vs, 0, kbits)
    t_ss = time.perf_counter() - t0
    return {"value": k.size / t_par, "unit": "records/s", "cores": cores, "kind": "oracle",
            "sample": f"{k.size} records ({'the full workload' if n_full else 'a slice'}, {dist_name}), stable LSD "
                      f"radix sort on {cores} host threads (oracle/cpu_baseline.cc, byte-identical to the oracle), "
                      f"{t_par:.2f} s",
            "host_model": oracle.host_model(),
            "oracle_1core": {"value": ns / t_or, "records": ns, "s": t_or,
                             "what": "oracle/oracle.c single-threaded LSD (64-bit words)"},
            "stable_sort_1core": {"value": ns / t_ss, "records": ns, "s": t_ss, "what": "std::stable_sort, 1 thread"}}


def _self_launch(args, argv) -> int | None:
    """`bench.py --gpus N` without torchrun's environment: start N ranks of this script
    with torch.distributed.run (one process per GPU, 127.0.0.1 rendezvous) and return its
    exit code; under torchrun, check that --gpus agrees with WORLD_SIZE."""
    ws = os.environ.get("WORLD_SIZE")
    if ws is not None:
        if int(ws) != args.gpus:
            sys.stderr.write(f"bench.py: --gpus {args.gpus} but WORLD_SIZE={ws}\n")
            raise SystemExit(2)
        return None
    if args.gpus <= 1:
        return None
    import socket
    with socket.socket() as sk:
        sk.bind(("127.0.0.1", 0))
        port = sk.getsockname()[1]
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={args.gpus}",
           "--master-addr", "127.0.0.1", "--master-port", str(port), os.path.abspath(__file__),
           *(argv if argv is not None else sys.argv[1:])]
    return subprocess.call(cmd)


def main(argv=None):
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="hrs", choices=["hrs", "reference"])
    ap.add_argument("--config", default="c2", choices=sorted(CONFIGS))
    ap.add_argument("--dist", default="uniform", choices=["uniform", "and2", "and3", "and4", "const"])
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--force-dist", action="store_true",
                    help="run the distributed path (NCCL) even at world size 1 (tests the N>1 code path on one GPU)")
    ap.add_argument("--exchange", default="grouped", choices=["grouped", "fused", "a2a"],
                    help="distributed exchange: bucket-major NCCL P2P (default), the fused scatter into the "
                         "receivers' buffers (CUDA IPC / NVLink peer memory, SURVEY N2), or one all-to-all")
    ap.add_argument("--nccl-timeout", type=int, default=300, help="seconds before a stuck collective aborts")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--cpu-log2", type=int, default=24)
    ap.add_argument("--ref-log2", type=int, default=24)
    args = ap.parse_args(argv)
    if args.warmup < 3:
        args.warmup = 3
    rc = _self_launch(args, argv)
    if rc is not None:
        return rc
    if args.impl == "reference":
        return run_reference(args)
    return run_hrs(args)


if __name__ == "__main__":
    sys.exit(main())
