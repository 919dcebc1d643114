"""Does a candidate's pass time depend on the kernel that ran before it?  On the bench image
(16384^2), time K=13 candidates back to back (the tuner's batches) and interleaved with a
K=11 pass (as bench.py's step loop runs them); per-pass CUDA events, median of 10.
    python tools/interleave_check.py [--k 13] [--prev 11] [--cands tma0,tma0s8,tma1,tma2]"""
import argparse
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--k", type=int, default=13)
ap.add_argument("--prev", type=int, default=11)
ap.add_argument("--cands", default="tma0,tma0s8,tma1,tma2,tma4")
a = ap.parse_args()
H = W = 16384
x = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 3)).cuda()
outs = {K: torch.empty((H - K + 1, W - K + 1), device="cuda") for K in (a.k, a.prev)}
plans = {K: sc.Plan(H, W, K) for K in (a.k, a.prev)}
prev_choice = plans[a.prev].tune(reps=10)
kern = {K: synth.binomial_kernel(K) for K in (a.k, a.prev)}


def choice(name):
    cfg = int(name.replace("tma", "").replace("s8", ""))
    return sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, 1 if name.endswith("s8") else 0)


def timed(run, interleave):
    ts = []
    for i in range(13):
        if interleave:
            plans[a.prev].run(x, kern[a.prev], outs[a.prev], "auto")
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        run()
        e1.record()
        if i >= 3:
            ts.append((e0, e1))
    torch.cuda.synchronize()
    return statistics.median(s.elapsed_time(e) * 1e3 for s, e in ts)


print("previous pass: K=%d %s" % (a.prev, prev_choice.name))
for name in a.cands.split(","):
    c = choice(name)
    run = (lambda c=c: plans[a.k].run_choice(x, kern[a.k], outs[a.k], c))
    print("K=%d %-16s back-to-back %7.1f us   after K=%d pass %7.1f us" %
          (a.k, c.name, timed(run, False), a.prev, timed(run, True)), flush=True)
