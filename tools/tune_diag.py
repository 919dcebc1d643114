"""Tuner diagnostics for the HBM-bound small widths at 16384^2: tune with SEPCONV_TUNE_LOG (every
candidate and every mutation child), then time chosen schedules back to back with run_choice.
Exploration only.
    SEPCONV_TUNE_LOG=gpurun_out/tune_diag.log python tools/tune_diag.py [--widths 3,5,7]"""
import argparse
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--size", type=int, default=16384)
    ap.add_argument("--widths", default="3,5,7")
    ap.add_argument("--batch", type=int, default=1, help="images per plan (BASELINE C5: 64 x 4096^2)")
    a = ap.parse_args()
    dev = torch.device("cuda", 0)
    H = W = a.size
    st = torch.cuda.current_stream(dev)
    img = torch.rand((a.batch, H, W), device=dev)
    for K in [int(x) for x in a.widths.split(",")]:
        p = sc.Plan(H, W, K, n=a.batch)
        out = torch.empty((a.batch, H - K + 1, W - K + 1), device=dev)
        k = synth.binomial_kernel(K)
        pick = p.tune(reps=10)
        print(f"K={K} tuner pick {pick.name} {pick.median_us:.1f} us", flush=True)
        trials = [pick]
        for cfg in range(6):
            for parts, grid in (((0, 0), (6, 96), (9, 144), (9, 148), (18, 148), (27, 148)) if a.batch == 1 else
                                ((0, 0), (1, 96), (1, 120), (1, 132), (1, 148), (2, 148))):
                trials.append(sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, 0, sched_parts=parts, sched_grid=grid))
        res = []
        for rnd in range(2):
            for c in trials:
                for _ in range(3):
                    p.run_choice(img, k, out, c, st)
                evs = []
                for _ in range(10):
                    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    e0.record(st)
                    p.run_choice(img, k, out, c, st)
                    e1.record(st)
                    evs.append((e0, e1))
                torch.cuda.synchronize()
                res.append((c.name, statistics.median(x.elapsed_time(y) * 1e3 for x, y in evs)))
        agg = {}
        for n, t in res:
            agg.setdefault(n, []).append(t)
        for t, n in sorted((min(v), n) for n, v in agg.items())[:12]:
            print(f"   {n:32s} {t:7.1f} us", flush=True)


if __name__ == "__main__":
    main()
