"""Sustained A/B timing of fused schedules (tail donation on/off) on one plan: a few seconds of
warm-up load, then interleaved back-to-back batches of every choice, repeated; the median and
min per choice.  Checks whether a schedule's burst advantage survives sustained power draw.
    python tools/steal_ab.py --size 16384 --k 17 --choices tma3,tma4@9:0:85,tma2@9:0:85"""
import argparse
import os
import statistics
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--size", type=int, default=16384)
ap.add_argument("--k", type=int, default=17)
ap.add_argument("--choices", default="tma3,tma4@9:0:85,tma2@9:0:85,tma4@18:0:0,tma2")
ap.add_argument("--rounds", type=int, default=15)
ap.add_argument("--n", type=int, default=10)
ap.add_argument("--warm", type=float, default=3.0)
a = ap.parse_args()
H = W = a.size
K = a.k
x = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 3)).cuda()
out = torch.empty((H - K + 1, W - K + 1), device="cuda")
k = synth.binomial_kernel(K)
p = sc.Plan(H, W, K)


def parse(spec):
    name, _, sch = spec.partition("@")
    cfg = int(name.replace("tma", "").replace("s8", ""))
    v = [int(t) for t in sch.split(":")] if sch else [0, 0, 0]
    v += [0] * (3 - len(v))
    return sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, 1 if name.endswith("s8") else 0,
                     sched_parts=v[0], sched_grid=v[1], sched_steal=v[2])


choices = [parse(s) for s in a.choices.split(",")]
ref = torch.empty_like(out)
p.run_choice(x, k, ref, choices[0])
for c in choices:                                      # same bits for every schedule
    p.run_choice(x, k, out, c)
    torch.cuda.synchronize()
    assert torch.equal(out, ref), c.name
t0 = time.time()
while time.time() - t0 < a.warm:
    for c in choices:
        p.run_choice(x, k, out, c)
    torch.cuda.synchronize()
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
ts = {c.name: [] for c in choices}
for r in range(a.rounds):
    for c in (choices if r % 2 == 0 else choices[::-1]):
        e0.record()
        for _ in range(a.n):
            p.run_choice(x, k, out, c)
        e1.record()
        torch.cuda.synchronize()
        ts[c.name].append(e0.elapsed_time(e1) * 1e3 / a.n)
for c in choices:
    v = ts[c.name]
    print("%5d K=%2d %-28s median %8.2f us  min %8.2f us" % (H, K, c.name, statistics.median(v), min(v)), flush=True)
