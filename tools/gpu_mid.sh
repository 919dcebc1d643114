#!/bin/bash
# Mid-size image investigation: precise cold/warm pass times and ncu captures.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r02}
timeout -s KILL 600 python tools/mid_timing.py ${MID_ARGS} > gpurun_out/${R}_mid_timing.json 2> gpurun_out/${R}_mid_timing.txt
echo "mid rc=$?"
for spec in ${PROF:-2048:17:sep-fused-tma2 2048:3:sep-fused-tma2 4096:17:sep-fused-tma2}; do
  S=${spec%%:*}; rest=${spec#*:}; K=${rest%%:*}; C=${rest#*:}
  timeout -s KILL 600 ncu --set full --clock-control none --import-source on -k regex:"stream_kernel|conv2d_kernel" -s 1 -c 1 \
    -o gpurun_out/${R}_${C}_s${S}_k${K} python tools/prof_one.py --size $S --k $K --cand $C --n 1 > gpurun_out/${R}_prof_${C}_s${S}_k${K}.log 2>&1
  echo "ncu $spec rc=$?"
done
ls -la gpurun_out
