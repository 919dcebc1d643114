"""Why does the bench time 16384^2 / K=17 at ~380 us when the tuner and tools/tune_diag.py time the
same candidate at ~352 us?  Replays the bench's K=17-only step (tuned AUTO, events around every
pass) while toggling one difference at a time: the nvidia-smi clock sampler, the input data
(synth.uniform_image vs torch.rand), the run path (sepconv_run vs run_choice), and the step count.
Exploration only.
    python tools/k17_probe.py"""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402


def main():
    dev = torch.device("cuda", 0)
    torch.cuda.set_device(dev)
    H = W = 16384
    K = int(os.environ.get("K17_PROBE_K", "17"))
    st = torch.cuda.current_stream(dev)
    img_synth = torch.from_numpy(synth.uniform_image(H, W, synth.BENCH_SEED_BASE + 3)).to(dev)
    img_rand = torch.rand((H, W), device=dev)
    out = torch.empty((H - K + 1, W - K + 1), device=dev)
    k = synth.binomial_kernel(K)
    p = sc.Plan(H, W, K)
    pick = p.tune(reps=10)
    print(f"K={K} tuner pick {pick.name} {pick.median_us:.1f} us", flush=True)

    def timed(img, n, use_choice, sampler):
        for _ in range(5):
            p.run(img, k, out, "auto", st)
        torch.cuda.synchronize()
        evs = []
        ctx = bench.ClockSampler(0) if sampler else None
        if ctx:
            ctx.__enter__()
        for _ in range(n):
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(st)
            if use_choice:
                p.run_choice(img, k, out, pick, st)
            else:
                p.run(img, k, out, "auto", st)
            b.record(st)
            evs.append((a, b))
        torch.cuda.synchronize()
        clk = None
        if ctx:
            ctx.__exit__(None, None, None)
            clk = ctx.summary()
        t = [x.elapsed_time(y) * 1e3 for x, y in evs]
        return statistics.mean(t), statistics.median(t), min(t), max(t), clk

    for rnd in range(2):
        for name, img, n, ch, smp in (("synth run 20", img_synth, 20, False, False),
                                      ("synth run 20 +sampler", img_synth, 20, False, True),
                                      ("rand run 20", img_rand, 20, False, False),
                                      ("synth choice 20", img_synth, 20, True, False),
                                      ("synth run 100", img_synth, 100, False, False),
                                      ("rand run 100 +sampler", img_rand, 100, False, True)):
            mean, med, lo, hi, clk = timed(img, n, ch, smp)
            print(f"  {name:24s} mean {mean:7.1f} median {med:7.1f} min {lo:7.1f} max {hi:7.1f} us  {clk or ''}",
                  flush=True)
    # the first passes of a run vs the last: is it a ramp?
    torch.cuda.synchronize()
    evs = []
    for _ in range(200):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        p.run(img_synth, k, out, "auto", st)
        b.record(st)
        evs.append((a, b))
    torch.cuda.synchronize()
    t = np.array([x.elapsed_time(y) * 1e3 for x, y in evs])
    print("  200 back-to-back passes, mean per block of 20:", " ".join(f"{v:.0f}" for v in t.reshape(10, 20).mean(1)))


if __name__ == "__main__":
    main()
