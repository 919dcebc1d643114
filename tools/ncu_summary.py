"""Summarise ncu captures (.ncu-rep) into profiles/: key metrics per kernel plus
profiles/traffic.json ({"<candidate>:K<k>": dram bytes per launch}) for bench.py's
roofline.traffic field.

    python tools/ncu_summary.py gpurun_out/r01_sep-fused-tma2_k3.ncu-rep ... --out profiles/r01_ncu_summary.md
File names must look like <round>_<candidate>_k<K>.ncu-rep.
"""
import argparse
import csv
import io
import json
import os
import re
import subprocess

METRICS = [
    ("gpu__time_duration.sum", "duration"),
    ("dram__bytes_read.sum", "DRAM read"),
    ("dram__bytes_write.sum", "DRAM write"),
    ("dram__throughput.avg.pct_of_peak_sustained_elapsed", "DRAM throughput % of peak"),
    ("lts__t_sectors_srcunit_tex_op_read.sum", "L2 read sectors (SM)"),
    ("l1tex__m_xbar2l1tex_read_bytes_mem_global_op_tma_ld.sum", "TMA load bytes"),
    ("l1tex__m_l1tex2xbar_write_bytes.sum", "L1->L2 write bytes"),
    ("sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active", "FMA pipe active %"),
    ("smsp__issue_active.avg.pct_of_peak_sustained_active", "issue active %"),
    ("smsp__inst_executed.sum", "instructions"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", "smem ld bank conflicts"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum", "smem st bank conflicts"),
    ("launch__registers_per_thread", "registers/thread"),
    ("launch__grid_size", "grid"),
    ("launch__block_size", "block"),
    ("sm__cycles_elapsed.avg.per_second", "SM clock"),
]


def raw(path):
    out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units, vals = rows[0], rows[1], rows[2]
    return {h: (v, u) for h, u, v in zip(hdr, units, vals)}


def to_bytes(v, u):
    x = float(v.replace(",", ""))
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}.get(u, 1)
    return x * scale


def stalls(m):
    items = []
    for k, (v, _) in m.items():
        if k.startswith("smsp__pcsamp_warps_issue_stalled_") and not k.endswith("not_issued"):
            try:
                items.append((float(v.replace(",", "")), k.replace("smsp__pcsamp_warps_issue_stalled_", "")))
            except ValueError:
                pass
    tot = sum(a for a, _ in items) or 1
    return ", ".join("%s %.0f%%" % (n, 100 * a / tot) for a, n in sorted(items, reverse=True)[:7])


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("reps", nargs="+")
    ap.add_argument("--out", required=True)
    ap.add_argument("--traffic", default="profiles/traffic.json")
    a = ap.parse_args()
    traffic = json.load(open(a.traffic)) if os.path.exists(a.traffic) else {}
    lines = ["# ncu --set full summaries (1 launch each, 16384^2 float32, --clock-control none)", ""]
    for path in a.reps:
        base = os.path.basename(path).replace(".ncu-rep", "")
        mt = re.match(r"r\d+_(.+)_k(\d+)$", base)
        cand, K = (mt.group(1), int(mt.group(2))) if mt else (base, 0)
        m = raw(path)
        lines.append("## %s, K=%d" % (cand, K))
        lines.append("")
        lines.append("| metric | value |")
        lines.append("|---|---|")
        for key, name in METRICS:
            if key in m:
                v, u = m[key]
                lines.append("| %s (`%s`) | %s %s |" % (name, key, v, u))
        rd, wr = m.get("dram__bytes_read.sum"), m.get("dram__bytes_write.sum")
        if rd and wr:
            tot = to_bytes(*rd) + to_bytes(*wr)
            alg = 4.0 * (16384 * 16384 + (16384 - K + 1) ** 2)
            lines.append("| DRAM read+write / algorithmic bytes | %.4f |" % (tot / alg))
            traffic["%s:K%d" % (cand, K)] = tot
        lines.append("| warp stall mix | %s |" % stalls(m))
        lines.append("")
    open(a.out, "w").write("\n".join(lines) + "\n")
    json.dump(traffic, open(a.traffic, "w"), indent=1, sort_keys=True)
    print("\n".join(lines))


if __name__ == "__main__":
    main()
