"""Turn an ncu launch-list CSV (--metrics gpu__time_duration.sum --csv) into the markdown
table kept under profiles/.

    python tools/launches_md.py gpurun_out/r01_launches.csv --bench profiles/r01_bench_v6.json \
        --out profiles/r01_ncu_launches_timed.md
"""
import argparse
import csv
import json

ap = argparse.ArgumentParser()
ap.add_argument("csv")
ap.add_argument("--bench", default="")
ap.add_argument("--out", required=True)
ap.add_argument("--cmd", default="python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline")
a = ap.parse_args()

with open(a.csv) as f:
    lines = [ln for ln in f if ln.startswith('"')]
rows = [r for r in csv.DictReader(lines) if r.get("Metric Name") == "gpu__time_duration.sum"]
total = sum(float(r["Metric Value"]) for r in rows) / 1e3
steps = 2
out = ["# ncu launch list of the timed region of `%s`" % a.cmd, "",
       "`ncu --metrics gpu__time_duration.sum --clock-control none --nvtx --nvtx-include \"sepconv_timed/\"` "
       "(cold-cache, serialised launches: compare shares, not absolutes).  %d launches." % len(rows), "",
       "| # | kernel | grid x block | us | share of step |", "|---|---|---|---|---|"]
for i, r in enumerate(rows):
    us = float(r["Metric Value"]) / 1e3
    name = r["Kernel Name"].replace("void ", "").split("(")[0]
    out.append("| %d | `%s` | %s x %s | %.1f | %.1f%% |" % (i, name, r["Grid Size"], r["Block Size"], us,
                                                          100 * us / (total / steps)))
out.append("")
line = "Total %.1f us for %d steps under ncu (%.1f us/step)" % (total, steps, total / steps)
if a.bench:
    d = json.load(open(a.bench))
    line += " (the same command printed %.0f us/step event-timed under ncu's serialised replay: not a bench value; `%s`)" % (d["ms_per_step"] * 1e3, a.bench)
out.append(line + ".")
open(a.out, "w").write("\n".join(out) + "\n")
print("\n".join(out[-3:]))
