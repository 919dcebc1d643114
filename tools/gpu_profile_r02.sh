#!/bin/bash
# Round-2 ncu evidence: (1) the launch list of bench.py's timed region (NVTX "sepconv_timed"),
# (2) DRAM bytes per launch of every fused candidate at every width (profiles/traffic.json),
# (3) full captures of chosen kernels, summarised on the box (reports are large).
#   PROF="17:sep-fused-tma3 9:sep-fused-tma0s8 3:sep-fused-tma2" bash tools/gpu_profile_r02.sh
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r02}
timeout -s KILL 900 ncu --metrics gpu__time_duration.sum --clock-control none --nvtx --nvtx-include "sepconv_timed/" \
   --csv --log-file gpurun_out/${R}_launches.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline \
   > gpurun_out/${R}_launches_bench.log 2>&1
echo "launch list rc=$?"
timeout -s KILL 1200 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
   -k regex:stream_kernel --csv --log-file gpurun_out/${R}_traffic.csv \
   python tools/traffic_all.py --order gpurun_out/${R}_traffic_order.json > gpurun_out/${R}_traffic.log 2>&1
echo "traffic rc=$?"
python tools/traffic_all.py --parse gpurun_out/${R}_traffic.csv --order gpurun_out/${R}_traffic_order.json \
   --out gpurun_out/traffic_fused.json >> gpurun_out/${R}_traffic.log 2>&1
for spec in ${PROF:-17:sep-fused-tma3 9:sep-fused-tma0s8 3:sep-fused-tma2}; do
  K=${spec%%:*}; C=${spec#*:}
  timeout -s KILL 900 ncu --set full --clock-control none --import-source on -k regex:"stream_kernel|conv2d_kernel" -s 1 -c 1 \
    -o gpurun_out/${R}_${C}_k${K} python tools/prof_one.py --k $K --cand $C --n 1 > gpurun_out/${R}_prof_${C}_k${K}.log 2>&1
  echo "full $spec rc=$?"
done
python tools/ncu_summary.py gpurun_out/${R}_*.ncu-rep --out gpurun_out/${R}_ncu_summary.md > gpurun_out/${R}_ncu_summary.log 2>&1
for f in gpurun_out/${R}_*.ncu-rep; do case "$f" in *${KEEP:-k17}.ncu-rep) ;; *) rm -f "$f";; esac; done
ls -la gpurun_out
