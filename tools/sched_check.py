"""Times fused candidates with explicit work-schedule overrides on one plan (device-resident,
back-to-back batches; clean-flushed batch differences when the working set fits in L2).
    python tools/sched_check.py --size 16384 --k 17 --cands tma2,tma3 --scheds 0:0,9:148,18:148,9:0:85
(a schedule is parts:grid[:steal], steal = the tail-donation percent)"""
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
ap.add_argument("--retime", action="store_true", help="with --tune: time the schedules again after tuning")
a = ap.parse_args()
H = W = a.size
K = a.k
x = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 3)).cuda()
out = torch.empty((H - K + 1, W - K + 1), device="cuda")
k = synth.binomial_kernel(K)
p = sc.Plan(H, W, K)
l2 = torch.cuda.get_device_properties(0).L2_cache_size
cold = 8 * H * W <= 2 * l2


def flush():
    sc.l2_flush()                                    # the bench's and the tuner's clean flush


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


def sweep(tag=""):
    for name in a.cands.split(","):
        cfg = int(name.replace("tma", "").replace("s8", ""))
        for sch in a.scheds.split(","):
            v = [int(t) for t in sch.split(":")] + [0]
            parts, grid, steal = v[0], v[1], v[2]
            c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, 1 if name.endswith("s8") else 0,
                          sched_parts=parts, sched_grid=grid, sched_steal=steal)
            print("%5d K=%2d %-14s parts %4d grid %4d steal %2d: %8.2f us%s" % (H, K, c.base_name, parts, grid, steal,
                                                                                 t_pass(c), tag), flush=True)


sweep()
if a.tune:
    for m in (-1, 12):
        b = p.tune(reps=10, force=True, mutations=m)
        print("tune(mutations=%d): %s %.2f us; re-timed %.2f us" % (m, b.name, b.median_us, t_pass(b)), flush=True)
    if a.retime:
        sweep("  (after tuning)")
