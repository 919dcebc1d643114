"""Overlap of the row-band halo exchange with the interior rows, measured on
the device with the library's band timeline (sepconv_band_trace / sepconv_band_timeline:
CUDA timing events around the interior kernel and the tail kernel on the compute stream and
around the NCCL send/recv group on the plan's comm stream; the phases are also NVTX ranges).

    python -m torch.distributed.run --nproc-per-node N --master-addr 127.0.0.1 \\
        tools/band_overlap.py [--size 16384] [--widths 3,9,17] [--reps 20]

Rank 0 prints one JSON line: per width and rank, the median interior / exchange / tail
intervals (ms from the call's start), the exchange time hidden under the interior kernel
(overlap / exchange duration) and the tail's share of the pass.  Needs N >= 2 GPUs (NCCL);
with one process it runs in external-halo mode (no exchange) as a smoke check."""
import argparse
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--size", type=int, default=16384)
    ap.add_argument("--widths", default="3,9,17")
    ap.add_argument("--reps", type=int, default=20)
    a = ap.parse_args()
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if world > 1:
        dist.init_process_group("nccl", device_id=dev)
        raw = sc.nccl_unique_id() if rank == 0 else bytes(sc.NCCL_ID_BYTES)
        t = torch.tensor(list(raw), dtype=torch.uint8, device=dev)
        dist.broadcast(t, 0)
        uid = bytes(t.cpu().tolist())
    else:
        uid = None
    H = W = a.size
    stream = torch.cuda.current_stream(dev)
    report = {"size": [H, W], "world": world, "widths": {}}
    for K in [int(x) for x in a.widths.split(",")]:
        r0, rows, owned, alloc = sc.band(H, K, world, rank)
        band = torch.empty((alloc, W), dtype=torch.float32, device=dev)
        band[:owned].copy_(torch.from_numpy(synth.uniform_image(H, W, synth.BENCH_SEED_BASE + 3,
                                                                rows=(r0, r0 + owned))))
        out = torch.empty((rows, W - K + 1), dtype=torch.float32, device=dev)
        p = sc.Plan(alloc, W, K, device=local)
        p.comm_init(uid, world, rank)
        p.tune(reps=5)
        p.band_trace(True)
        k = synth.binomial_kernel(K)
        phases = {"interior": [], "exchange": [], "tail": [], "total": [], "overlap": []}
        for i in range(a.reps + 3):
            p.run_band(band, k, out, "auto", stream)
            tl = p.band_timeline()
            if i < 3:
                continue
            (i0, i1), (x0, x1), (t0, t1) = tl["interior"], tl["exchange"], tl["tail"]
            phases["interior"].append(i1 - i0)
            phases["exchange"].append(x1 - x0)
            phases["tail"].append(t1 - t0)
            phases["total"].append(max(i1, x1, t1))
            phases["overlap"].append(max(0.0, min(i1, x1) - max(i0, x0)))
        med = {k_: statistics.median(v) for k_, v in phases.items()}
        row = {"interior_ms": med["interior"], "exchange_ms": med["exchange"], "tail_ms": med["tail"],
               "pass_ms": med["total"],
               "exchange_hidden": (med["overlap"] / med["exchange"]) if med["exchange"] > 0 else None,
               "tail_share": med["tail"] / med["total"] if med["total"] > 0 else None}
        rows_all = [None] * world
        if world > 1:
            dist.all_gather_object(rows_all, row)
        else:
            rows_all = [row]
        report["widths"][str(K)] = rows_all
        p.close()
    if rank == 0:
        print(json.dumps(report), flush=True)
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
