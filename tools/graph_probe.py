"""What would a CUDA graph buy the launch-bound legs?  Marginal device time after the clean flush
(bench.py CleanFlush / time_flushed) of one call issued directly and of the same call captured
once into a CUDA graph and replayed: Poisson2D SOR at the paper's 2048^2 (24 iterations, the
tuned multi-launch wavefront), Black-Scholes at the paper's 500 000 options, SeparableConvolution
at 2048^2 (K = 3, 17).  Exploration only.
    python tools/graph_probe.py"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_asplos_phothilimthanaara13_b200 import bs, sepconv as sc, sor, synth  # noqa: E402


def graphed(fn):
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        fn(s)                                   # warm: plans, tensor maps, first-call costs
    torch.cuda.current_stream().wait_stream(s)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        fn(torch.cuda.current_stream())
    torch.cuda.synchronize()
    return g


def main():
    dev = torch.device("cuda", 0)
    torch.cuda.set_device(dev)
    flush = bench.CleanFlush(torch, dev)
    st = torch.cuda.current_stream(dev)
    steps = 50

    def report(tag, direct, graph):
        d = min(bench.time_flushed(torch, st, steps, direct, flush) for _ in range(3))
        g = min(bench.time_flushed(torch, st, steps, graph.replay, flush) for _ in range(3))
        print(f"{tag:44s} direct {d * 1e3:8.2f} us   graph replay {g * 1e3:8.2f} us   ({(d - g) * 1e3:+.2f})", flush=True)

    # Poisson2D SOR, 2048^2, 24 iterations
    n, iters = 2048, 24
    x, b = synth.poisson_problem(n, n, seed=synth.BENCH_SEED_BASE + 40)
    omega = 2.0 / (1.0 + np.sin(np.pi / (n - 1)))
    p = sor.SorPlan(n, n)
    vid, depth = p.tune(iters_hint=iters, reps=3)
    p.load(torch.from_numpy(x).to(dev), torch.from_numpy(b).to(dev))
    torch.cuda.synchronize()
    report(f"SOR 2048^2 x24 (variant {vid}, depth {depth})", lambda: p.iterate(omega, iters, "auto", st),
           graphed(lambda s: p.iterate(omega, iters, "auto", s)))
    for dep in (3, 6):
        p.set_depth(dep)
        report(f"SOR 2048^2 x24 wave depth {dep}", lambda: p.iterate(omega, iters, "wave", st),
               graphed(lambda s: p.iterate(omega, iters, "wave", s)))
    report("SOR 2048^2 x24 half-sweeps (48 launches)", lambda: p.iterate(omega, iters, "half", st),
           graphed(lambda s: p.iterate(omega, iters, "half", s)))

    # Black-Scholes, 500 000 options
    m = 500000
    s_, x_, t_ = (torch.from_numpy(a).to(dev) for a in synth.bs_options(m, seed=synth.BENCH_SEED_BASE + 50))
    c_, q_ = torch.empty_like(s_), torch.empty_like(s_)
    report("Black-Scholes 500000", lambda: bs.price(s_, x_, t_, synth.BS_RATE, synth.BS_VOL, c_, q_, stream=st),
           graphed(lambda s: bs.price(s_, x_, t_, synth.BS_RATE, synth.BS_VOL, c_, q_, stream=s)))

    # SeparableConvolution, 2048^2
    H = W = 2048
    img = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE)).to(dev)
    for K in (3, 17):
        k = synth.binomial_kernel(K)
        out = torch.empty((H - K + 1, W - K + 1), device=dev)
        pl = sc.Plan(H, W, K)
        pl.tune()
        report(f"sepconv 2048^2 K={K} auto", lambda: pl.run(img, k, out, "auto", st),
               graphed(lambda s: pl.run(img, k, out, "auto", s)))


if __name__ == "__main__":
    main()
