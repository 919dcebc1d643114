"""Sub-microsecond pass times for mid-size images despite the ~2 us granularity of CUDA events
on this system (profiles/r02_flush_study.txt shows medians snapping to multiples of 2.048 us).

    python tools/mid_timing.py [--sizes 64,2048,3520,4096] [--widths 3,17] [--n 200] [--only a,b]

Per (size, K, candidate): events around N iterations of [clean flush, pass] and around N
iterations of [clean flush] alone; pass = difference / N.  "clean flush" = write 2 x L2, then
read a second 2 x L2 buffer, so the pass starts with an L2 of clean unrelated lines.  Also the
L2-warm steady state: events around N back-to-back passes (no host sync), / N.
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
    ap.add_argument("--sizes", default="64,2048,3520,4096")
    ap.add_argument("--widths", default="3,17")
    ap.add_argument("--n", type=int, default=200)
    ap.add_argument("--only", default="")
    a = ap.parse_args()
    l2 = torch.cuda.get_device_properties(0).L2_cache_size
    wbuf = torch.empty(2 * l2 // 4, device="cuda")
    rbuf = torch.ones(2 * l2 // 4, device="cuda")
    sink = torch.empty((), device="cuda")
    only = set(a.only.split(",")) if a.only else None

    def flush():
        wbuf.fill_(1.0)
        torch.sum(rbuf, dim=0, out=sink)

    def timed(fn, n):
        fn()
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for _ in range(n):
            fn()
        e1.record()
        torch.cuda.synchronize()
        return e0.elapsed_time(e1) * 1e3 / n

    res = {}
    t_flush = timed(flush, a.n)
    res["flush_us"] = t_flush
    print("clean flush alone %.2f us" % t_flush, file=sys.stderr, flush=True)
    for H in [int(x) for x in a.sizes.split(",")]:
        img = torch.from_numpy(synth.uniform_image(H, H, seed=synth.BENCH_SEED_BASE + 2)).cuda()
        for K in [int(x) for x in a.widths.split(",")]:
            if K > H:
                continue
            k = synth.binomial_kernel(K)
            p = sc.Plan(H, H, K)
            out = torch.empty((H - K + 1, H - K + 1), device="cuda")
            for c in p.candidates():
                if only and c.name not in only:
                    continue
                run = (lambda c=c: p.run_choice(img, k, out, c))
                tf = timed(flush, a.n)
                tfp = timed(lambda: (flush(), run()), a.n)
                tw = timed(run, a.n)
                cold = tfp - tf
                mb = 8.0 * H * H / 1e6
                res["%d/%d/%s" % (H, K, c.name)] = {"cold_us": cold, "warm_us": tw, "flush_us": tf}
                print("%5d K=%-2d %-20s cold %7.2f us (%5.0f GB/s)  warm %7.2f us" %
                      (H, K, c.name, cold, mb * 1e3 / cold, tw), file=sys.stderr, flush=True)
    print(json.dumps(res))


if __name__ == "__main__":
    main()
