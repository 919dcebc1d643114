"""Black-Scholes leg of bench.py (`python bench.py --workload blackscholes`), SURVEY.md 8(f)
NEXT-4: the paper's elementwise benchmark (test input 500000 options, Fig. 8
P:949).  Not the headline metric (BASELINE.json names SeparableConvolution).

A "step" = pricing `--options` options (default 2^28: 5.4 GB of compulsory traffic, far
larger than L2) resident in HBM.  value = options of the whole job per second (N ranks each
price their own shard: no exchange, weak scaling).  e2e = bs_price_host on pinned host
buffers.  cpu_baseline = the double oracle on a bounded sample."""
from __future__ import annotations

import json
import os
import statistics
import time

import numpy as np

from paper_conf_asplos_phothilimthanaara13_b200 import synth

ROOT = os.path.dirname(os.path.abspath(__file__))

METRIC = "Black-Scholes European options priced per second (Moptions/s)"


def _oracle_sample(target_s: float):
    import oracle
    n = 1 << 16
    s, x, t = synth.bs_options(n, seed=synth.BENCH_SEED_BASE + 50)
    t0 = time.perf_counter()
    oracle.black_scholes(s, x, t, synth.BS_RATE, synth.BS_VOL)
    probe = max(time.perf_counter() - t0, 1e-4)
    reps = int(max(1, min(200, target_s / probe)))
    t0 = time.perf_counter()
    for _ in range(reps):
        oracle.black_scholes(s, x, t, synth.BS_RATE, synth.BS_VOL)
    el = time.perf_counter() - t0
    return {"value": n * reps / el / 1e6, "unit": "Moptions/s", "cores": 1, "kind": "oracle",
            "sample": f"{reps} x {n} options (oracle_black_scholes, double, one thread), {el:.1f} s"}


def bs_config(n, world, flush, flush_label):
    """The workload's `config`, identical for the CUDA arm and the reference arm."""
    return {"workload": f"Black-Scholes, {n} float32 options per GPU (r={synth.BS_RATE}, v={synth.BS_VOL})",
            "options": n, "l2": flush_label if flush else "inputs larger than L2 (no flush)",
            "parallelism": f"options sharded x{world}" if world > 1 else "1 GPU"}


def run(args, peaks_fn, dist_env, ClockSampler, emit, flushing=None, l2_bytes=126 * 2 ** 20):
    world, rank, local = dist_env()
    if args.impl == "reference":
        if rank != 0:
            return 0
        vals, last = [], None
        for i in range(args.warmup + args.steps):
            last = _oracle_sample(max(1.0, 40.0 / max(1, args.steps + args.warmup)))
            if i >= args.warmup:
                vals.append(last["value"])
        v = statistics.median(vals)
        emit({"impl": "reference", "metric": METRIC, "value": v, "unit": "Moptions/s",
              "n_gpus": world if world > 1 else args.gpus,
              "steps": args.steps, "warmup": args.warmup, "higher_is_better": True, "scaling": "weak",
              "vs_baseline": None, "dtype": "f64", "data": "synthetic",
              # the CUDA arm's config, key for key (the oracle times a sample: cpu_baseline.sample)
              "config": bs_config(args.options, world, 20 * args.options <= 2 * l2_bytes, flushing[0].LABEL),
              "cpu_baseline": {"value": v, "unit": "Moptions/s", "cores": 1, "kind": "oracle", "sample": last["sample"]},
              "e2e": {"value": v, "unit": "Moptions/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}})
        return 0

    import torch
    from paper_conf_asplos_phothilimthanaara13_b200 import bs
    from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc

    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist = None
    if world > 1:
        import torch.distributed as dist
        dist.init_process_group("nccl", device_id=dev)
    peak_gbs, peak_src = peaks_fn()
    n = args.options
    s, x, t = synth.bs_options(n, seed=synth.BENCH_SEED_BASE + 50 + rank)
    ds, dx, dt = (torch.from_numpy(a).to(dev) for a in (s, x, t))
    dc = torch.empty(n, dtype=torch.float32, device=dev)
    dp = torch.empty(n, dtype=torch.float32, device=dev)
    stream = torch.cuda.current_stream(dev)
    r, v = synth.BS_RATE, synth.BS_VOL
    for _ in range(max(args.warmup, 0)):
        bs.price(ds, dx, dt, r, v, dc, dp, stream=stream)
    torch.cuda.synchronize()
    if dist:
        dist.barrier()
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(args.steps)]
    # a working set that fits in L2 (the paper's 500000 options: 10 MB) gets a clean flush before
    # every step and is timed as a batched difference (bench.py CleanFlush / time_flushed)
    l2_bytes = torch.cuda.get_device_properties(dev).L2_cache_size or 126 * 2 ** 20
    flush = 20 * n <= 2 * l2_bytes
    CleanFlush, time_flushed = flushing
    flusher = CleanFlush(torch, dev) if flush else None
    launches0 = sc.launch_count()
    with ClockSampler(local) as clk:
        torch.cuda.synchronize()
        torch.cuda.nvtx.range_push("sepconv_timed")
        if flush:
            ms = time_flushed(torch, stream, args.steps,
                              lambda: bs.price(ds, dx, dt, r, v, dc, dp, stream=stream), flusher)
        else:
            for i in range(args.steps):
                ev[i][0].record(stream)
                bs.price(ds, dx, dt, r, v, dc, dp, stream=stream)
                ev[i][1].record(stream)
        torch.cuda.nvtx.range_pop()
        torch.cuda.synchronize()
    launches = sc.launch_count() - launches0
    if not flush:
        ms = statistics.median(a.elapsed_time(b) for a, b in ev)
    if dist:
        tt = torch.tensor([ms], dtype=torch.float64, device=dev)
        dist.all_reduce(tt, op=dist.ReduceOp.MAX)
        ms = float(tt[0])
    value = n * world / (ms * 1e-3) / 1e6
    byts = 20.0 * n
    achieved = byts / (ms * 1e-3) / 1e9
    traffic = None                       # ncu DRAM read + write bytes of one launch (profiles/traffic.json)
    try:
        traffic = json.load(open(os.path.join(ROOT, "profiles", "traffic.json"))).get(f"bs_kernel_vec:n{n}")
    except Exception:
        traffic = None
    roofline = {"bound": "hbm", "kernel": "bs_kernel_vec", "achieved": achieved, "peak": peak_gbs, "unit": "GB/s",
                "frac": achieved / peak_gbs, "traffic": traffic, "peak_source": peak_src,
                "algorithmic_bytes_per_launch": byts, "algorithmic": "20 B per option (S, X, T read; call, put written)"}
    e2e = None
    if not args.no_e2e:
        hs, hx, ht = (torch.from_numpy(a).pin_memory() for a in (s, x, t))
        hc = torch.empty(n, dtype=torch.float32).pin_memory()
        hp = torch.empty(n, dtype=torch.float32).pin_memory()
        bs.price_host(hs, hx, ht, r, v, hc, hp, stream=stream)
        t0 = time.perf_counter()
        reps = 2
        for _ in range(reps):
            bs.price_host(hs, hx, ht, r, v, hc, hp, stream=stream)
        el = (time.perf_counter() - t0) / reps
        if dist:
            tt = torch.tensor([el], dtype=torch.float64, device=dev)
            dist.all_reduce(tt, op=dist.ReduceOp.MAX)
            el = float(tt[0])
        e2e = {"value": n * world / el / 1e6, "unit": "Moptions/s", "h2d_bytes_per_step": 12 * n,
               "d2h_bytes_per_step": 8 * n, "ms_per_step": el * 1e3,
               "api": "bs_price_host (pinned host buffers, two-stream chunk pipeline)"}
    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cpu = _oracle_sample(args.cpu_seconds)
    if rank == 0:
        emit({"metric": METRIC, "value": value, "unit": "Moptions/s", "n_gpus": world, "steps": args.steps,
              "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "weak",
              "vs_baseline": None, "dtype": "f32", "data": "synthetic",
              "config": bs_config(n, world, flush, CleanFlush.LABEL),
              "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": int(launches),
              "clocks": clk.summary()})
    if dist:
        dist.barrier()
        dist.destroy_process_group()
    return 0
