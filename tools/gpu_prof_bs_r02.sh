#!/bin/bash
# ncu evidence for the round-2 Black-Scholes kernel (plain grid, bs_kernel_vec<1>) on 2^28 options:
# DRAM bytes + duration of one launch, and one --set full capture summarised on the box.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
timeout -s KILL 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
   -k regex:bs_kernel -s 1 -c 1 --csv --log-file gpurun_out/r02_bs_traffic.csv python tools/prof_bs.py > gpurun_out/r02_bs_traffic.log 2>&1
echo "traffic rc=$?"
timeout -s KILL 900 ncu --set full --clock-control none --import-source on -k regex:bs_kernel -s 1 -c 1 \
   -o gpurun_out/r02_bs_full python tools/prof_bs.py > gpurun_out/r02_bs_full.log 2>&1
echo "full rc=$?"
python tools/ncu_summary.py gpurun_out/r02_bs_full.ncu-rep --out gpurun_out/r02_bs_ncu_summary.md > gpurun_out/r02_bs_ncu_summary.log 2>&1
rm -f gpurun_out/r02_bs_full.ncu-rep
cat gpurun_out/r02_bs_traffic.csv | tail -4; cat gpurun_out/r02_bs_ncu_summary.md | head -40
