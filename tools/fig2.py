"""The paper's Fig. 2 re-run on B200: execution time of every mapping of
SeparableConvolution vs kernel width, plus the tuner's pick.

    python tools/fig2.py [--size 3520] [--widths 3,5,...,17] [--reps 20] > profiles/r01_fig2_3520.json

Mappings (the paper's four: 2D / Separable x local memory / no local memory)
are the C ABI's candidates: 2d-direct, 2d-tma, sep-unfused-direct, sep-unfused-tma, plus
the B200-only fused separable kernels (sep-fused-*).  Times are device times (CUDA events;
when the working set fits in L2, the marginal time after the clean flush sepconv_l2_flush, as
bench.py measures it, R25); the paper's
include PCIe copies, so only the shape of the curves is comparable.
"""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc  # noqa: E402
from paper_conf_asplos_phothilimthanaara13_b200 import synth  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--size", type=int, default=3520)
    ap.add_argument("--widths", default="3,5,7,9,11,13,15,17")
    ap.add_argument("--reps", type=int, default=20)
    ap.add_argument("--md", default="", help="also append a markdown table of the sweep to this file")
    a = ap.parse_args()
    H = W = a.size
    img = torch.from_numpy(synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 2)).cuda()
    stream = torch.cuda.current_stream()
    cold = 8 * H * W <= 2 * torch.cuda.get_device_properties(0).L2_cache_size
    res = {"size": [H, W], "widths": {}, "unit": "us",
           "timing": ("marginal pass time after sepconv_l2_flush (clean flush): events around %d x [flush, pass] minus "
                      "%d x [flush], median of 3" % (a.reps, a.reps)) if cold else
                     "events around %d back-to-back passes, median of 3" % a.reps}

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

    def pass_us(run):
        ts = []
        for _ in range(3):
            if cold:
                ts.append(batch(lambda: (sc.l2_flush(stream), run()), a.reps) - batch(lambda: sc.l2_flush(stream), a.reps))
            else:
                ts.append(batch(run, a.reps))
        return sorted(ts)[1]

    for K in [int(x) for x in a.widths.split(",")]:
        k = synth.binomial_kernel(K)
        p = sc.Plan(H, W, K)
        out = torch.empty((H - K + 1, W - K + 1), device="cuda")
        row = {}
        for c in p.candidates():
            row[c.name] = pass_us(lambda c=c: p.run_choice(img, k, out, c))
        best = p.tune(reps=a.reps)
        row["tuner"] = {"pick": best.name, "us": best.median_us}
        res["widths"][str(K)] = row
        print(K, {n: round(v, 1) for n, v in row.items() if n != "tuner"}, row["tuner"], file=sys.stderr)
    print(json.dumps(res))
    if a.md:
        widths = list(res["widths"])
        names = [n for n in res["widths"][widths[0]] if n != "tuner"]
        lines = ["## %d² float32 (%s)" % (H, res["timing"]), "",
                 "| mapping | " + " | ".join("K=%s" % k for k in widths) + " |",
                 "|---|" + "---|" * len(widths)]
        for n in names:
            lines.append("| %s | " % n + " | ".join("%.1f" % res["widths"][k][n] if n in res["widths"][k] else "–"
                                                   for k in widths) + " |")
        lines.append("| **tuner pick** | " + " | ".join("%s (%.1f)" % (res["widths"][k]["tuner"]["pick"],
                                                                       res["widths"][k]["tuner"]["us"])
                                                      for k in widths) + " |")
        with open(a.md, "a") as f:
            f.write("\n".join(lines) + "\n\n")


if __name__ == "__main__":
    main()
