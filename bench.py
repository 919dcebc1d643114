#!/usr/bin/env python3
"""bench.py -- SeparableConvolution on B200: output Mpixels/s and HBM GB/s per kernel width.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
                    [--workload image|batch] [--widths 3,5,...,17]

Workload (BASELINE.json configs[3], the metric's configuration): one 16384 x 16384
float32 image, kernel widths K = 3, 5, ..., 17.  A "step" is one SeparableConvolution
of the image per width (8 passes of the whole hot path), each with the tuned AUTO
variant.  At N > 1 (torchrun) the image is split into N row bands, one per GPU, and
every pass exchanges the (K-1)-row halo with NCCL send/recv inside the C ABI
(sepconv_run_band); scaling is strong (fixed image).  --workload batch is
configs[4] (64 x 4096^2, K = 11, images sharded over ranks, no exchange).  --workload
poisson is the NEXT-3 Poisson2D red-black SOR leg (bench_poisson.py), --workload
blackscholes the NEXT-4 Black-Scholes leg (bench_bs.py).

value = output pixels of the whole job per step / max-over-ranks device time
(CUDA events, inputs resident in HBM; the 1.07 GB image is larger than the 126 MB
L2, so no flush is needed between steps).  e2e = the same metric through
sepconv_run_host with pinned HOST buffers, copies inside the timed region.
The oracle (oracle/, test infrastructure) runs only in the cpu_baseline leg and in
--impl reference, on a bounded sample, on rank 0.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

from paper_conf_asplos_phothilimthanaara13_b200 import synth  # noqa: E402

METRIC = "output Mpixels/s and HBM GB/s (% of B200 peak) per kernel width, 1/2/4/8 GPUs"
HBM_FALLBACK_GBS = 6650.0          # /opt/skills/guides/B200_PROFILING.md fallback (used only if MEASURED_PEAKS.json is absent)
NOMINAL_HBM_GBS = 8000.0           # BASELINE.json north_star "roughly 8 TB/s"


def parse_args():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--workload", choices=["image", "batch", "poisson", "blackscholes"], default="image")
    ap.add_argument("--widths", default="3,5,7,9,11,13,15,17")
    ap.add_argument("--size", type=int, default=16384, help="image side (image workload)")
    ap.add_argument("--variant", default="auto")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--cpu-seconds", type=float, default=12.0, help="target oracle time for the cpu_baseline sample")
    ap.add_argument("--tune-reps", type=int, default=10)
    ap.add_argument("--tune-mutations", type=int, default=0,
                    help="schedule mutations after the exhaustive tuning pass (0 = library default 12, -1 = none)")
    ap.add_argument("--sor-iters", type=int, default=24, help="poisson workload: iterations per step")
    ap.add_argument("--options", type=int, default=1 << 28, help="blackscholes workload: options per GPU")
    ap.add_argument("--dry-run", action="store_true",
                    help="launcher/protocol check without a GPU: N ranks on gloo exchange the halo rows of "
                         "their bands (no convolution runs, value is null)")
    return ap.parse_args()


def peaks():
    path = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        with open(path) as f:
            d = json.load(f)
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs: torch D2D copy)"
    except Exception:
        return HBM_FALLBACK_GBS, "fallback (B200_PROFILING.md)"


def _free_port() -> int:
    import socket
    with socket.socket(socket.AF_INET, socket.SOCK_STREAM) as so:
        so.bind(("127.0.0.1", 0))
        return so.getsockname()[1]


def spawn_ranks(args):
    """`bench.py --gpus N` outside torchrun: launch N ranks (one process per GPU) through
    torch.distributed.run on 127.0.0.1 and return their exit status.  Never measures fewer
    GPUs than asked: too few devices, or a WORLD_SIZE that disagrees with --gpus, is an error.
    Returns None when this process is already the rank it should be."""
    env_world = os.environ.get("WORLD_SIZE")
    if env_world is not None:
        if int(env_world) != args.gpus and args.impl != "reference":
            print(f"[bench] error: --gpus {args.gpus} but WORLD_SIZE={env_world}", file=sys.stderr)
            return 2
        return None
    if args.gpus <= 1 or args.impl == "reference":
        return None
    if not args.dry_run:
        import torch
        have = torch.cuda.device_count()
        if have < args.gpus:
            print(f"[bench] error: --gpus {args.gpus} but this node has {have} CUDA device(s)", file=sys.stderr)
            return 2
    env = dict(os.environ)
    if not args.dry_run:                 # NCCL reports nranks when each communicator comes up
        env.setdefault("NCCL_DEBUG", "INFO")
        env.setdefault("NCCL_DEBUG_SUBSYS", "INIT")
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={args.gpus}",
           "--master-addr=127.0.0.1", f"--master-port={_free_port()}", os.path.abspath(__file__), *sys.argv[1:]]
    print(f"[bench] launching {args.gpus} ranks: {' '.join(cmd)}", file=sys.stderr, flush=True)
    return subprocess.call(cmd, env=env)


def dist_env():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


class ClockSampler:
    """nvidia-smi clocks + throttle reasons during the timed region (B200_PROFILING.md recipe)."""
    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index = index
        self.proc = None
        self.file = tempfile.NamedTemporaryFile("w+", suffix=".csv", delete=False)

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.index), "--query-gpu=" + self.FIELDS,
                                          "--format=csv,noheader,nounits", "-lms", "100"],
                                         stdout=self.file, stderr=subprocess.DEVNULL)
            time.sleep(0.3)
        except Exception:
            self.proc = None
        return self

    def __exit__(self, *exc):
        if self.proc:
            time.sleep(0.25)
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except Exception:
                self.proc.kill()

    def summary(self):
        if not self.proc:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        self.file.flush()
        rows = []
        with open(self.file.name) as f:
            for line in f:
                parts = [p.strip() for p in line.split(",")]
                if len(parts) < 9:
                    continue
                try:
                    rows.append((float(parts[1]), float(parts[2]), float(parts[3]), parts[5:9]))
                except ValueError:
                    continue
        os.unlink(self.file.name)
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["no samples"]}
        loaded = [r for r in rows if r[2] > 200] or rows
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i, v in enumerate(r[3]) if v.lower().startswith("active")})
        return {"sm_mhz": statistics.median(r[0] for r in loaded), "sm_max_mhz": max(r[1] for r in rows),
                "power_w_max": max(r[2] for r in rows), "samples": len(rows), "reasons": reasons}


# --------------------------------------------------------------------------------------------
class CleanFlush:
    """The L2 flush between timed passes when the working set fits in L2: sepconv_l2_flush, which
    writes a 2 x L2 buffer and then reads a second 2 x L2 buffer, so the pass starts from an L2
    of clean, unrelated lines (a write alone leaves ~L2-size of dirty lines whose write-back the
    next pass would pay, profiles/r02_flush_study.txt).  The tuner times its candidates after the
    same flush, so its picks and this bench see the same conditions."""

    def __init__(self, torch, dev):
        from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
        self.sc = sc
        self.stream = torch.cuda.current_stream(dev)
        for i in range(3):                       # first-call costs stay out of any timing
            self(i)

    def __call__(self, i=0):
        self.sc.l2_flush(self.stream)

    LABEL = ("L2 flushed before every step (sepconv_l2_flush: write 2 x L2, then read another 2 x L2 so L2 holds "
             "clean unrelated lines); step time = [events around steps x (flush + step)] - [mean of events around steps x flush "
             "before and after], / steps, after a spin-up of 20 flushes")


def time_flushed(torch, stream, steps, body, flush):
    """Marginal device ms of `body` after a clean flush: events around `steps` x [flush, body]
    minus the mean of event-timed `steps` x [flush] batches run just before and just after it
    (single event pairs around a short pass read a ~5 us event/launch floor in 2.048 us ticks,
    profiles/r02_latency_probe.txt).  A spin-up of flushes first brings the clocks up from idle,
    so the first batch is not timed on a ramping GPU."""
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(6)]
    for i in range(20):
        flush(i)
    ev[0].record(stream)
    for i in range(steps):
        flush(i)
    ev[1].record(stream)
    ev[2].record(stream)
    for i in range(steps):
        flush(i)
        body()
    ev[3].record(stream)
    ev[4].record(stream)
    for i in range(steps):
        flush(i)
    ev[5].record(stream)
    torch.cuda.synchronize()
    t_flush = 0.5 * (ev[0].elapsed_time(ev[1]) + ev[4].elapsed_time(ev[5]))
    return max(1e-6, ev[2].elapsed_time(ev[3]) - t_flush) / steps


# --------------------------------------------------------------------------------------------
def oracle_sample(img_rows_fn, W, widths, target_s, nthreads=0, H=None):
    """Time the oracle (as it stands) on the first S output rows of the image for every width;
    an image with fewer rows than the sample needs is convolved whole, `reps` times over."""
    import oracle
    cores = nthreads or oracle.num_cpus()
    kmax = max(widths)
    max_rows = (H - kmax + 1) if H else 8192

    def run(S, reps=1):
        src = img_rows_fn(S + kmax - 1)
        t0 = time.perf_counter()
        px = 0
        for _ in range(reps):
            for K in widths:
                out = oracle.convolve2d(np.ascontiguousarray(src[:S + K - 1]), synth.binomial_kernel(K),
                                        nthreads=cores)
                px += out.size
        return time.perf_counter() - t0, px

    S0 = min(16, max_rows)
    t_probe, _ = run(S0)
    want = int(S0 * target_s / max(t_probe, 1e-5))
    S = int(max(S0, min(8192, max_rows, want)))
    reps = max(1, min(100000, want // max(S, 1))) if S == max_rows else 1
    t, px = run(S, reps)
    if S == max_rows and t < 0.5 * target_s:          # tiny images: the probe was overhead-bound
        reps = max(1, min(1000000, int(reps * target_s / max(t, 1e-5))))
        t, px = run(S, reps)
    what = (f"the whole image x {reps}" if reps > 1 or S == max_rows else f"first {S} output rows")
    return {"value": px / t / 1e6, "unit": "Mpixels/s", "cores": cores, "kind": "oracle",
            "sample": f"{what} ({S} output rows x {W - min(widths) + 1}..{W - kmax + 1} cols), "
                      f"widths {widths[0]}..{widths[-1]} (K^2 double MACs/px), {t:.1f} s",
            "seconds": t, "pixels": px}


def emit(d):
    print(json.dumps(d), flush=True)


def l2_bytes_of(dev=None):
    """The device's L2 size (the flush rule); 126 MiB (B200) when no device is visible."""
    try:
        import torch
        if torch.cuda.is_available():
            return torch.cuda.get_device_properties(dev or 0).L2_cache_size or 126 * 2 ** 20
    except Exception:
        pass
    return 126 * 2 ** 20


def image_config(args, world, H, W, N_img, widths, seed, flush):
    """The image / batch workload's `config`, identical for the CUDA arm and the reference arm."""
    return {"workload": (f"{H}x{W} float32 image, kernel widths {','.join(map(str, widths))}, one pass per width"
                         if args.workload == "image" else f"{N_img} x {H}x{W} float32 images, width 11"),
            "image": [H, W], "images": N_img, "widths": widths, "variant": args.variant + " (tuned per width)",
            "kernel": "normalised binomial C(K-1,i)/2^(K-1)", "seed": seed,
            "l2": (CleanFlush.LABEL.replace("step", "pass") + "; per width; ms_per_step = sum over widths")
            if flush else "inputs larger than L2 (no flush)",
            "parallelism": (f"row bands x{world}, NCCL halo send/recv" if world > 1 and args.workload == "image"
                            else f"images sharded x{world}" if world > 1 else "1 GPU")}


# --------------------------------------------------------------------------------------------
def run_reference(args):
    """--impl reference: the oracle (the paper's definition in plain C, double) on host cores."""
    world, rank, _ = dist_env()
    if rank != 0:
        return 0
    widths = [int(x) for x in args.widths.split(",")] if args.workload == "image" else [11]
    W = args.size if args.workload == "image" else 4096
    H = W
    seed = synth.BENCH_SEED_BASE + (3 if args.workload == "image" else 4)
    # each step a bounded sample: about a minute for the whole --steps/--warmup run, at most
    # --cpu-seconds per step (tests pass a small value)
    per_step_s = max(0.2, min(args.cpu_seconds, 60.0 / max(1, args.steps + args.warmup)))
    rows_cache = {}

    def img_rows(n):
        if n not in rows_cache:
            rows_cache[n] = synth.uniform_image(H, W, seed, rows=(0, min(H, n)))
        return rows_cache[n]

    for _ in range(args.warmup):
        oracle_sample(img_rows, W, widths, per_step_s / 4, H=H)
    vals, times = [], []
    last = None
    for _ in range(args.steps):
        last = oracle_sample(img_rows, W, widths, per_step_s, H=H)
        vals.append(last["value"])
        times.append(last["seconds"])
    value = statistics.median(vals)
    # the same workload string and keys as the CUDA arm's line (the oracle times a sample of it)
    # the CUDA arm's config, key for key (the oracle times a bounded sample of it: cpu_baseline.sample)
    N_img = 1 if args.workload == "image" else 64
    cfg = image_config(args, world, H, W, N_img, widths, seed,
                       8 * H * W * N_img // max(world, 1) <= 2 * l2_bytes_of())
    emit({"impl": "reference", "metric": METRIC, "value": value, "unit": "Mpixels/s",
          "n_gpus": world if world > 1 else args.gpus,
          "steps": args.steps, "warmup": args.warmup, "ms_per_step": statistics.median(times) * 1e3,
          "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "f64",
          "data": "synthetic", "config": cfg,
          "cpu_baseline": {"value": value, "unit": "Mpixels/s", "cores": last["cores"], "kind": "oracle",
                           "sample": last["sample"]},
          "e2e": {"value": value, "unit": "Mpixels/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}})
    return 0


# --------------------------------------------------------------------------------------------
def run_dry(args):
    """--dry-run: the multi-rank plumbing of the image workload without a GPU.  Every rank takes
    its row band from sepconv_band (host arithmetic of libsepconv.so), fills its owned input rows
    from the seeded generator, receives the K-1 halo rows from rank g+1 over gloo (the exchange
    sepconv_run_band does with NCCL) and checks them against the generator.  No convolution runs;
    rank 0 prints the JSON line with value null."""
    import torch
    import torch.distributed as dist
    from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
    world, rank, _ = dist_env()
    if world > 1:
        dist.init_process_group("gloo")
    H = W = args.size
    seed = synth.BENCH_SEED_BASE + 3
    widths = [int(x) for x in args.widths.split(",")]
    halo_ok = True
    halo_bytes = 0
    for K in widths:
        r0, rows, owned, alloc = sc.band(H, K, world, rank)
        band = np.zeros((alloc, W), np.float32)
        band[:owned] = synth.uniform_image(H, W, seed, rows=(r0, r0 + owned))
        if world > 1:
            ops = []
            if rank > 0:                            # my first K-1 rows are the predecessor's halo
                ops.append(dist.P2POp(dist.isend, torch.from_numpy(np.ascontiguousarray(band[:K - 1])), rank - 1))
            recv = torch.empty((alloc - owned, W), dtype=torch.float32)
            if rank < world - 1 and alloc > owned:
                ops.append(dist.P2POp(dist.irecv, recv, rank + 1))
            for w_ in (dist.batch_isend_irecv(ops) if ops else []):
                w_.wait()
            if rank < world - 1 and alloc > owned:
                band[owned:] = recv.numpy()
                halo_bytes += recv.numel() * 4
        want = synth.uniform_image(H, W, seed, rows=(r0, r0 + alloc))
        halo_ok &= bool(np.array_equal(band, want))
    flags = torch.tensor([0 if halo_ok else 1, halo_bytes], dtype=torch.int64)
    if world > 1:
        dist.all_reduce(flags)
    if rank == 0:
        emit({"metric": METRIC, "value": None, "unit": "Mpixels/s", "n_gpus": world, "steps": 0,
              "warmup": 0, "ms_per_step": None, "higher_is_better": True, "scaling": "strong",
              "vs_baseline": None, "dtype": "f32", "data": "synthetic", "dry_run": True,
              "halo_exchange_ok": int(flags[0]) == 0, "halo_bytes": int(flags[1]),
              "config": {"workload": f"{H}x{W} float32 image, kernel widths {','.join(map(str, widths))}, "
                                     "one pass per width", "widths": widths,
                         "parallelism": f"row bands x{world}, gloo halo send/recv (dry run)"}})
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()
    return 0 if int(flags[0]) == 0 else 1


def main():
    args = parse_args()
    rc = spawn_ranks(args)
    if rc is not None:
        return rc
    if args.dry_run:
        return run_dry(args)
    if args.workload == "poisson":
        import bench_poisson
        return bench_poisson.run(args, peaks, dist_env, ClockSampler, emit, (CleanFlush, time_flushed), l2_bytes_of())
    if args.workload == "blackscholes":
        import bench_bs
        return bench_bs.run(args, peaks, dist_env, ClockSampler, emit, (CleanFlush, time_flushed), l2_bytes_of())
    if args.impl == "reference":
        return run_reference(args)

    import torch
    from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc

    world, rank, local = dist_env()
    if world != args.gpus:
        print(f"[bench] error: --gpus {args.gpus} but WORLD_SIZE={world}", file=sys.stderr)
        return 2
    print(f"[bench] rank {rank}/{world} on cuda:{local}", file=sys.stderr, flush=True)
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist = None
    if world > 1:
        import torch.distributed as dist
        dist.init_process_group("nccl", device_id=dev)

    peak_gbs, peak_src = peaks()
    widths = [int(x) for x in args.widths.split(",")]
    if args.workload == "batch":
        widths = [11]
        N_img, H = 64, 4096
        W = H
    else:
        N_img, H = 1, args.size
        W = H
    seed = synth.BENCH_SEED_BASE + (3 if args.workload == "image" else 4)
    stream = torch.cuda.current_stream(dev)

    # ---- this rank's share of the input, resident in HBM ----
    if args.workload == "image":
        bands = {K: sc.band(H, K, world, rank) for K in widths}
        kmax = max(widths)
        # one buffer holding the union of the bands' rows (bands shift slightly with K)
        r_lo = min(b[0] for b in bands.values())
        r_hi = max(b[0] + b[3] for b in bands.values())
        host_img = synth.uniform_image(H, W, seed, rows=(r_lo, min(H, r_hi)))
        dev_img = torch.empty((r_hi - r_lo + kmax, W), dtype=torch.float32, device=dev)
        dev_img[:host_img.shape[0]].copy_(torch.from_numpy(host_img))
        plans, outs, ins = {}, {}, {}
        uid = None
        if world > 1:                                   # one NCCL communicator shared by every width's plan
            raw = sc.nccl_unique_id() if rank == 0 else bytes(sc.NCCL_ID_BYTES)
            t = torch.tensor(list(raw), dtype=torch.uint8, device=dev)
            dist.broadcast(t, 0)
            uid = bytes(t.cpu().tolist())
        for K in widths:
            r0, rows, owned, alloc = bands[K]
            p = sc.Plan(alloc, W, K, device=local)
            if world > 1:
                p.comm_init(uid, world, rank)
            plans[K] = p
            outs[K] = torch.empty((rows, W - K + 1), dtype=torch.float32, device=dev)
            # the band's own input rows; rows past `owned` are the halo, written by run_band
            ins[K] = dev_img[r0 - r_lo:r0 - r_lo + alloc]
            if world > 1:
                ins[K] = ins[K].clone()     # run_band writes the halo rows: keep bands private per width
        out_px_rank = {K: outs[K].numel() for K in widths}
        out_px_job = {K: (H - K + 1) * (W - K + 1) for K in widths}
        in_rows_job = {K: H for K in widths}
    else:
        per = N_img // world
        n0 = rank * per
        host_img = np.stack([synth.uniform_image(H, W, seed, n=n0 + i) for i in range(per)])
        dev_img = torch.from_numpy(host_img).to(dev)
        K = widths[0]
        plans = {K: sc.Plan(H, W, K, n=per, device=local)}
        outs = {K: torch.empty((per, H - K + 1, W - K + 1), dtype=torch.float32, device=dev)}
        ins = {K: dev_img}
        out_px_rank = {K: outs[K].numel()}
        out_px_job = {K: N_img * (H - K + 1) * (W - K + 1)}
        in_rows_job = {K: N_img * H}

    kernels = {K: synth.binomial_kernel(K) for K in widths}

    # ---- tune (the paper's install-time autotuning): per width, per rank ----
    choices = {}
    for K in widths:
        choices[K] = plans[K].tune(reps=args.tune_reps, mutations=args.tune_mutations)
    torch.cuda.synchronize()
    if world > 1:
        # every rank runs rank 0's pick (sepconv_set_choice): the step ends with the slowest rank,
        # and per-rank picks made under tuning noise would let the worst of them set the pace
        for K in widths:
            c = choices[K]
            t = torch.tensor([c.algo, c.mapping, c.fused, c.config, c.store_path, c.sched_parts, c.sched_grid,
                              c.sched_steal], dtype=torch.int64, device=dev)
            dist.broadcast(t, 0)
            if rank != 0:
                v = [int(x) for x in t.tolist()]
                plans[K].set_choice(sc.Choice(v[0], v[1], v[2], v[3], v[4], sched_parts=v[5], sched_grid=v[6],
                                              sched_steal=v[7]))
                choices[K] = plans[K].get_choice("auto")
    l2_bytes = torch.cuda.get_device_properties(dev).L2_cache_size or 126 * 2 ** 20
    flush = max(8 * (H * W * N_img) // max(world, 1), 0) <= 2 * l2_bytes

    def one_pass(K):
        if world > 1 and args.workload == "image":
            plans[K].run_band(ins[K], kernels[K], outs[K], args.variant, stream)
        else:
            plans[K].run(ins[K], kernels[K], outs[K], args.variant, stream)

    # ---- warm-up ----
    for _ in range(max(args.warmup, 0)):
        for K in widths:
            one_pass(K)
    torch.cuda.synchronize()
    if dist:
        dist.barrier()

    # ---- timed region: CUDA events on the launching stream ----
    # Inputs larger than L2 (the default 16384^2, the batch) run the steps back to back: events
    # around every pass and around the whole timed region.  Working sets that fit in L2 (in + out
    # <= 2 x L2: 2048^2-4096^2) need a flush before every pass: a write of a 2 x L2 scratch buffer,
    # then a read of a second 2 x L2 buffer, so the pass starts from an L2 of clean, unrelated
    # lines (a write alone leaves ~L2-size of dirty lines whose write-back the pass would pay:
    # +2-6 us, profiles/r02_flush_study.txt).  A single event pair around one short pass measures
    # a ~5 us event/launch floor in 2.048 us ticks (profiles/r02_latency_probe.txt), so per
    # width the flushed mode times `steps` x [flush, pass] and `steps` x [flush] between event
    # pairs and takes the difference (time_flushed): the marginal device time of the pass inside
    # a stream of work, as the unflushed mode measures it.
    do_flush = CleanFlush(torch, dev) if flush else None

    def evpair():
        return torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)

    ev = {K: [evpair() for _ in range(args.steps)] for K in widths}
    per_k_ms = {}
    e_start, e_end = evpair()
    launches0 = sc.launch_count()
    with ClockSampler(local) as clk:
        torch.cuda.synchronize()
        if dist:
            dist.barrier()
        torch.cuda.nvtx.range_push("sepconv_timed")      # ncu --nvtx-include sepconv_timed/
        e_start.record(stream)
        if flush:
            for K in widths:
                per_k_ms[K] = time_flushed(torch, stream, args.steps, lambda K=K: one_pass(K), do_flush)
        else:
            for s in range(args.steps):
                for K in widths:
                    ev[K][s][0].record(stream)
                    one_pass(K)
                    ev[K][s][1].record(stream)
        e_end.record(stream)
        torch.cuda.nvtx.range_pop()
        torch.cuda.synchronize()
        if dist:
            dist.barrier()
    launches = sc.launch_count() - launches0
    if dist:
        tl = torch.tensor([launches], dtype=torch.int64, device=dev)
        dist.all_reduce(tl)
        launches = int(tl.item())
    if flush:                                    # the flushes are not part of the step
        total_ms = sum(per_k_ms.values()) * args.steps
    else:
        total_ms = e_start.elapsed_time(e_end)
        per_k_ms = {K: sum(a.elapsed_time(b) for a, b in ev[K]) / args.steps for K in widths}
    if dist:
        t = torch.tensor([total_ms] + [per_k_ms[K] for K in widths], dtype=torch.float64, device=dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        total_ms = float(t[0])
        per_k_ms = {K: float(t[1 + i]) for i, K in enumerate(widths)}
    ms_per_step = total_ms / args.steps
    px_step = sum(out_px_job.values())
    value = px_step / (ms_per_step * 1e-3) / 1e6

    # algorithmic bytes: read every input once, write every output once, + received halo
    def alg_bytes(K):
        b = 4 * (in_rows_job[K] * W + out_px_job[K])
        if world > 1 and args.workload == "image":
            b += 4 * (K - 1) * W * (world - 1)
        return b

    per_width = {}
    for K in widths:
        t_s = per_k_ms[K] * 1e-3
        gbs = alg_bytes(K) / t_s / 1e9
        per_width[str(K)] = {"variant": choices[K].name, "tuned_us": choices[K].median_us,
                             "us": per_k_ms[K] * 1e3, "mpix_s": out_px_job[K] / t_s / 1e6, "gbs": gbs,
                             "frac_of_measured": gbs / (peak_gbs * world),
                             "frac_of_8tbs": gbs / (NOMINAL_HBM_GBS * world)}

    # roofline for the dominant kernel (the compiled candidate with the largest share of the step;
    # a tuned work-schedule override "@p..g.." is a launch parameter of the same kernel)
    def kname(K):
        return per_width[str(K)]["variant"].split("@")[0]
    names = [kname(K) for K in widths]
    dom = max(set(names), key=lambda n: sum(per_k_ms[K] for K in widths if kname(K) == n))
    dom_k = [K for K in widths if kname(K) == dom]
    dom_bytes = sum(alg_bytes(K) for K in dom_k) / world          # per GPU, per launch set
    dom_s = sum(per_k_ms[K] for K in dom_k) * 1e-3
    achieved = dom_bytes / dom_s / 1e9
    traffic = None
    tr_path = os.path.join(ROOT, "profiles", "traffic.json")
    if os.path.exists(tr_path):
        try:
            tr = json.load(open(tr_path))
            base = dom                                     # ncu traffic is per candidate, any schedule
            vals = [tr[f"{base}:K{K}"] for K in dom_k if f"{base}:K{K}" in tr and args.workload == "image"
                    and world == 1 and H == 16384]
            if len(vals) == len(dom_k):
                traffic = sum(vals) / len(vals)
        except Exception:
            traffic = None
    roofline = {"bound": "hbm", "kernel": dom, "widths": dom_k, "achieved": achieved, "peak": peak_gbs,
                "unit": "GB/s", "frac": achieved / peak_gbs, "traffic": traffic, "peak_source": peak_src,
                "algorithmic_bytes_per_launch": dom_bytes / len(dom_k),
                "frac_of_8tbs": achieved / NOMINAL_HBM_GBS}
    if dom_bytes < 256e6:
        # a pass moving this little is bound by launch latency, pipeline fill and the K-1 warm-up
        # rows of short segments (~5 us fixed per pass, profiles/r01_small_latency.txt), not by HBM
        roofline["note"] = ("latency-bound: the pass moves %.1f MB; a fixed ~5 us per pass (launch, first TMA "
                            "round trip, store drain) dominates, so frac is not an HBM-efficiency figure"
                            % (dom_bytes / len(dom_k) / 1e6))

    # ---- e2e: the public API with pinned HOST buffers, copies inside the timed region ----
    e2e = None
    if not args.no_e2e:
        e2e_steps = max(1, min(args.steps, 2))
        h_out = {}
        hplans = {}
        if args.workload == "image":
            bands = {K: sc.band(H, K, world, rank) for K in widths}
            h_in = torch.from_numpy(host_img).pin_memory()
            for K in widths:
                r0, rows, owned, alloc = bands[K]
                hplans[K] = sc.Plan(alloc, W, K, device=local)
                hplans[K].tune(reps=3)
                h_out[K] = torch.empty((rows, W - K + 1), dtype=torch.float32).pin_memory()
        else:
            h_in = torch.from_numpy(host_img).pin_memory()
            K = widths[0]
            hplans[K] = plans[K]
            h_out[K] = torch.empty(tuple(outs[K].shape), dtype=torch.float32).pin_memory()
        h2d = d2h = 0

        def e2e_pass(K):
            nonlocal h2d, d2h
            if args.workload == "image":
                r0, rows, owned, alloc = bands[K]
                src = h_in[r0 - r_lo:r0 - r_lo + alloc]
                hplans[K].run_host(src, kernels[K], h_out[K], args.variant, stream)
                h2d += src.numel() * 4
            else:
                hplans[K].run_host(h_in, kernels[K], h_out[K], args.variant, stream)
                h2d += h_in.numel() * 4
            d2h += h_out[K].numel() * 4

        for K in widths:
            e2e_pass(K)
        h2d = d2h = 0
        torch.cuda.synchronize()
        if dist:
            dist.barrier()
        t0 = time.perf_counter()
        for _ in range(e2e_steps):
            for K in widths:
                e2e_pass(K)
        torch.cuda.synchronize()
        el = time.perf_counter() - t0
        if dist:
            t = torch.tensor([el, h2d, d2h], dtype=torch.float64, device=dev)
            tmax = t.clone()
            dist.all_reduce(tmax, op=dist.ReduceOp.MAX)
            dist.all_reduce(t, op=dist.ReduceOp.SUM)
            el, h2d, d2h = float(tmax[0]), float(t[1]), float(t[2])
        e2e = {"value": px_step * e2e_steps / el / 1e6, "unit": "Mpixels/s",
               "h2d_bytes_per_step": int(h2d / e2e_steps), "d2h_bytes_per_step": int(d2h / e2e_steps),
               "ms_per_step": el / e2e_steps * 1e3, "api": "sepconv_run_host (pinned host buffers)"}

    # ---- cpu_baseline: the oracle as it stands, bounded sample, rank 0 at N=1 only ----
    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        if args.workload == "image":
            cpu = oracle_sample(lambda n: host_img[:n], W, widths, args.cpu_seconds, H=H)
        else:
            cpu = oracle_sample(lambda n: host_img[0][:n], W, widths, args.cpu_seconds, H=H)
        cpu = {k: v for k, v in cpu.items() if k not in ("seconds", "pixels")}
        if args.workload == "image" and H <= 256:
            # the small case also reports the single-thread oracle
            one = oracle_sample(lambda n: host_img[:n], W, widths, min(args.cpu_seconds, 3.0), nthreads=1, H=H)
            cpu["single_thread"] = {"value": one["value"], "unit": "Mpixels/s", "cores": 1, "sample": one["sample"]}

    if rank == 0:
        cfg = image_config(args, world, H, W, N_img, widths, seed, flush)
        emit({"metric": METRIC, "value": value, "unit": "Mpixels/s", "n_gpus": world, "steps": args.steps,
              "warmup": args.warmup, "ms_per_step": ms_per_step, "higher_is_better": True, "scaling": "strong",
              "vs_baseline": None, "dtype": "f32", "data": "synthetic", "config": cfg,
              "hbm_gbs": sum(alg_bytes(K) for K in widths) / (ms_per_step * 1e-3) / 1e9,
              "per_width": per_width, "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e,
              "gpu_launches": int(launches), "clocks": clk.summary(),
              "tuning": f"sepconv_tune per width (reps {args.tune_reps}; flushed when the inputs fit in L2, else "
                        "back to back)"})
    if dist:
        dist.barrier()
        dist.destroy_process_group()
    return 0


if __name__ == "__main__":
    sys.exit(main())
