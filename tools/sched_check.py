"""Times fused candidates with explicit work-schedule overrides on one plan (device-resident,
back-to-back batches; clean-flushed batch differences when the working set fits in L2).
    python tools/sched_check.py --size 16384 --k 17 --cands tma2,tma3 --scheds 0:0,9:148,18:148"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--size", type=int, default=16384)
ap.add_argument("--k", type=int, default=17)
ap.add_argument("--cands", default="tma2,tma3")
ap.add_argument("--scheds", default="0:0,9:148,9:0,18:148,5:74")
ap.add_argument("--n", type=int, default=10)
ap.add_argument("--tune", action="store_true")
a = ap.parse_args()
H = W = a.size
K = a.k
x = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 3)).cuda()
out = torch.empty((H - K + 1, W - K + 1), device="cuda")
k = synth.binomial_kernel(K)
p = sc.Plan(H, W, K)
l2 = torch.cuda.get_device_properties(0).L2_cache_size
cold = 8 * H * W <= 2 * l2
wb = torch.empty(2 * l2 // 4, device="cuda")
rb = torch.zeros(2 * l2 // 4, device="cuda")
sink = torch.empty((), device="cuda")


def flush():
    wb.fill_(1.0)
    torch.sum(rb, dim=0, out=sink)


def batch(fn, n):
    fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(n):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) * 1e3 / n


def t_pass(c):
    run = lambda: p.run_choice(x, k, out, c)  # noqa: E731
    ts = []
    for _ in range(3):
        ts.append(batch(lambda: (flush(), run()), a.n) - batch(flush, a.n) if cold else batch(run, a.n))
    return sorted(ts)[1]


for name in a.cands.split(","):
    cfg = int(name.replace("tma", "").replace("s8", ""))
    for sch in a.scheds.split(","):
        parts, grid = (int(v) for v in sch.split(":"))
        c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, 1 if name.endswith("s8") else 0, sched_parts=parts,
                      sched_grid=grid)
        print("%5d K=%2d %-14s parts %4d grid %4d: %8.2f us" % (H, K, c.base_name, parts, grid, t_pass(c)), flush=True)
if a.tune:
    for m in (-1, 12):
        b = p.tune(reps=10, force=True, mutations=m)
        print("tune(mutations=%d): %s %.2f us; re-timed %.2f us" % (m, b.name, b.median_us, t_pass(b)), flush=True)
