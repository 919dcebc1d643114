"""Does the tuner's per-width pick survive the bench's step (all widths back to back, sustained
power)?  Tunes every width of the 16384^2 bench as bench.py does, then times every fused TMA
candidate of each width INSIDE the step (the other widths run their current picks), and finally
compares whole steps with the tuner's picks against steps with the in-step winners, interleaved.
Exploration only.
    python tools/insitu_probe.py [--size 16384] [--widths 3,5,...,17] [--steps 5]"""
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
    ap.add_argument("--widths", default="3,5,7,9,11,13,15,17")
    ap.add_argument("--steps", type=int, default=5)
    a = ap.parse_args()
    dev = torch.device("cuda", 0)
    torch.cuda.set_device(dev)
    H = W = a.size
    widths = [int(x) for x in a.widths.split(",")]
    st = torch.cuda.current_stream(dev)
    img = torch.from_numpy(synth.uniform_image(H, W, synth.BENCH_SEED_BASE + 3)).to(dev)
    plans = {K: sc.Plan(H, W, K) for K in widths}
    outs = {K: torch.empty((H - K + 1, W - K + 1), device=dev) for K in widths}
    ks = {K: synth.binomial_kernel(K) for K in widths}
    picks = {K: plans[K].tune(reps=10) for K in widths}
    cands = {}
    for K in widths:
        seen, lst = set(), []
        for c in [picks[K]] + [c for c in plans[K].candidates()
                               if c.algo == sc.SEPCONV_SEPARABLE and c.fused and c.mapping == sc.MAP_TMA]:
            if c.key() not in seen:
                seen.add(c.key())
                lst.append(c)
        cands[K] = lst
    cur = dict(picks)

    def steps(n, choice):
        evs = {K: [] for K in widths}
        for _ in range(n):
            for K in widths:
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(st)
                plans[K].run_choice(img, ks[K], outs[K], choice[K], st)
                e1.record(st)
                evs[K].append((e0, e1))
        torch.cuda.synchronize()
        return {K: [x.elapsed_time(y) * 1e3 for x, y in evs[K]] for K in widths}

    steps(10, cur)                                     # warm-up into the sustained state
    best = {}
    for K in widths:
        res = []
        for rnd in range(2):                           # two interleaved rounds over the candidates
            for c in cands[K]:
                ch = dict(cur)
                ch[K] = c
                t = steps(a.steps, ch)[K]
                res.append((c.name, statistics.median(t)))
        agg = {}
        for n, t in res:
            agg.setdefault(n, []).append(t)
        ranked = sorted(((min(v), n) for n, v in agg.items()))
        tuned_t = min(agg[picks[K].name])
        best[K] = next(c for c in cands[K] if c.name == ranked[0][1])
        print(f"K={K:2d} tuned {picks[K].name:28s} (tuner {picks[K].median_us:6.1f} us) in-step {tuned_t:6.1f} us | "
              + "  ".join(f"{n}:{t:.1f}" for t, n in ranked[:4]), flush=True)
    # whole steps, interleaved blocks
    tot = {"tuned": [], "in-step": []}
    for blk in range(6):
        for name, ch in (("tuned", picks), ("in-step", best)):
            t = steps(a.steps, ch)
            tot[name].append(sum(statistics.median(t[K]) for K in widths))
    for name, v in tot.items():
        px = sum((H - K + 1) * (W - K + 1) for K in widths)
        m = statistics.median(v)
        print(f"{name:8s} step {m:8.1f} us  ({px / m:.0f} Mpx/s)  blocks: " + " ".join(f"{x:.0f}" for x in v))


if __name__ == "__main__":
    main()
