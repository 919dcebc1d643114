"""Poisson2D SOR variants on one B200: cell-updates/s and pass bandwidth per variant/depth.

    python tools/sor_perf.py [--sizes 2048,16384] [--iters 24] [--reps 5]

HALF moves 16 B per cell per iteration (two in-place half-sweeps: read own colour, b and
the other colour, write own colour); WAVE depth T moves 12 B per cell per pass of T
iterations (read u, b once, write u once) plus the halo-strip overlap."""
import argparse
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch

from paper_conf_asplos_phothilimthanaara13_b200 import sor, synth

ap = argparse.ArgumentParser()
ap.add_argument("--sizes", default="2048,8192,16384")
ap.add_argument("--iters", type=int, default=24)
ap.add_argument("--reps", type=int, default=5)
ap.add_argument("--depths", default="1,2,3,4,5,6,8")
a = ap.parse_args()

for size in [int(v) for v in a.sizes.split(",")]:
    n = m = size
    x = torch.rand((n, m), device="cuda")
    b = torch.rand((n, m), device="cuda") * (1.0 / (n - 1) ** 2)
    p = sor.SorPlan(n, m)
    p.load(x, b)
    omega = synth.omega_opt(n, m)
    cands = [("half", 0)] + [("wave", int(d)) for d in a.depths.split(",")]
    for v, d in cands:
        p.set_depth(d)
        ts = []
        for r in range(a.reps + 1):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            torch.cuda.synchronize()
            e0.record()
            p.iterate(omega, a.iters, v)
            e1.record()
            torch.cuda.synchronize()
            if r:
                ts.append(e0.elapsed_time(e1) * 1e-3)
        t = statistics.median(ts)
        cells = n * m * a.iters
        byts = n * m * (16.0 * a.iters if v == "half" else 12.0 * (-(-a.iters // d)))
        print(f"{size:6d}^2 {v:4s} T={d}  {t * 1e3:9.3f} ms  {cells / t / 1e9:8.1f} Gcell-it/s  "
              f"{byts / t / 1e9:7.0f} GB/s (variant bytes)", flush=True)
    p.close()
    del x, b
    torch.cuda.empty_cache()
