"""How the L2 flush between timed passes changes the measured time of mid-size images.

    python tools/flush_study.py [--sizes 2048,3520,4096] [--widths 3,7,11,15,17] [--reps 15]

For every candidate of every (size, K) plan, the median device time (CUDA events around the
one pass) under three regimes:
  write   : the scratch fill of 2 x L2 that bench.py used in round 1 -- leaves ~L2-size of
            DIRTY lines, whose write-back the timed pass then pays while it allocates lines
  clean   : the same write, then a read of a second 2 x L2 buffer -- L2 ends full of clean,
            unrelated lines: the pass starts cold and pays only its own traffic
  warm    : no flush, back-to-back passes (in + out may stay L2-resident: not a HBM number)
Prints one JSON object (per size, K, candidate: the three medians) and a table on stderr.
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
    ap.add_argument("--sizes", default="2048,3520,4096")
    ap.add_argument("--widths", default="3,7,11,15,17")
    ap.add_argument("--reps", type=int, default=15)
    ap.add_argument("--only", default="", help="comma list of candidate names (default: all)")
    a = ap.parse_args()
    l2 = torch.cuda.get_device_properties(0).L2_cache_size
    wbuf = torch.empty(2 * l2 // 4, device="cuda")
    rbuf = torch.ones(2 * l2 // 4, device="cuda")
    sink = torch.empty((), device="cuda")
    only = set(a.only.split(",")) if a.only else None

    def flush(mode):
        if mode in ("write", "clean"):
            wbuf.fill_(1.0)
        if mode == "clean":
            torch.sum(rbuf, dim=0, out=sink)

    res = {"l2_bytes": l2, "reps": a.reps, "sizes": {}}
    for H in [int(x) for x in a.sizes.split(",")]:
        img = torch.from_numpy(synth.uniform_image(H, H, seed=synth.BENCH_SEED_BASE + 2)).cuda()
        res["sizes"][str(H)] = {}
        for K in [int(x) for x in a.widths.split(",")]:
            k = synth.binomial_kernel(K)
            p = sc.Plan(H, H, K)
            out = torch.empty((H - K + 1, H - K + 1), device="cuda")
            row = {}
            for c in p.candidates():
                if only and c.name not in only:
                    continue
                t = {}
                for mode in ("write", "clean", "warm"):
                    ts = []
                    for r in range(a.reps + 3):
                        flush(mode)
                        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                        e0.record()
                        p.run_choice(img, k, out, c)
                        e1.record()
                        torch.cuda.synchronize()
                        if r >= 3:
                            ts.append(e0.elapsed_time(e1) * 1e3)
                    ts.sort()
                    t[mode] = ts[len(ts) // 2]
                row[c.name] = t
                print(H, K, "%-22s" % c.name, " ".join("%s %7.1f" % (m, v) for m, v in t.items()), file=sys.stderr,
                      flush=True)
            res["sizes"][str(H)][str(K)] = row
    print(json.dumps(res))


if __name__ == "__main__":
    main()
