"""DRAM traffic per launch of every fused-separable candidate at every benchmark width.

    ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum \
        --clock-control none -k regex:stream_kernel --csv --log-file gpurun_out/traffic.csv \
        python tools/traffic_all.py --order gpurun_out/traffic_order.json
    python tools/traffic_all.py --parse gpurun_out/traffic.csv --order gpurun_out/traffic_order.json \
        --out profiles/traffic.json

The first form launches, on the bench's 16384^2 image, every fused candidate once per width
(K = 3, 5, ..., 17) and writes the launch order; the second joins the ncu rows to that order
and writes {"<candidate>:K<k>": dram read + write bytes per launch} for bench.py's
roofline.traffic (so the field is filled whichever candidate the tuner picks on the day).
"""
import argparse
import csv
import io
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def launch(order_path, size, widths):
    import torch
    from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth
    x = torch.rand((size, size), device="cuda")
    order = []
    for K in widths:
        out = torch.empty((size - K + 1, size - K + 1), device="cuda")
        with sc.Plan(size, size, K) as p:
            k = synth.binomial_kernel(K)
            for c in p.candidates():
                if not c.name.startswith("sep-fused"):
                    continue
                p.run_choice(x, k, out, c)
                torch.cuda.synchronize()
                order.append([c.name, K])
        del out
    with open(order_path, "w") as f:
        json.dump(order, f)
    print("launched", len(order))


def parse(csv_path, order_path, out_path):
    text = open(csv_path).read()
    start = text.find('"ID"')
    rows = list(csv.DictReader(io.StringIO(text[start:])))
    by_id = {}
    for r in rows:
        d = by_id.setdefault(r["ID"], {"name": r["Kernel Name"]})
        v = float(r["Metric Value"].replace(",", ""))
        unit = r.get("Metric Unit", "")
        scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9}.get(unit, 1)
        d[r["Metric Name"]] = v * scale if "bytes" in r["Metric Name"] else v
    launches = [by_id[i] for i in sorted(by_id, key=int) if "stream_kernel" in by_id[i]["name"]]
    order = json.load(open(order_path))
    assert len(launches) == len(order), (len(launches), len(order))
    traffic = {}
    for (cand, K), d in zip(order, launches):
        traffic[f"{cand}:K{K}"] = d["dram__bytes_read.sum"] + d["dram__bytes_write.sum"]
    with open(out_path, "w") as f:
        json.dump(dict(sorted(traffic.items())), f, indent=1)
    print("wrote", out_path, len(traffic))


if __name__ == "__main__":
    ap = argparse.ArgumentParser()
    ap.add_argument("--order", required=True)
    ap.add_argument("--parse")
    ap.add_argument("--out")
    ap.add_argument("--size", type=int, default=16384)
    ap.add_argument("--widths", default="3,5,7,9,11,13,15,17")
    a = ap.parse_args()
    if a.parse:
        parse(a.parse, a.order, a.out)
    else:
        launch(a.order, a.size, [int(k) for k in a.widths.split(",")])
