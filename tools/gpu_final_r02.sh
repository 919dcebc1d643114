#!/bin/bash
# Round-2 final evidence on one fresh box: the driver's GPU tests and smoke, every bench leg,
# the Fig. 2 sweep, the ncu launch list of bench.py's timed region and two full captures.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r02z}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.limit --format=csv > gpurun_out/${R}_nvsmi.txt 2>&1
timeout -s KILL 1500 python -m pytest tests -x -q -m gpu > gpurun_out/${R}_pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/${R}_pytest_gpu.log
timeout -s KILL 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${R}_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/${R}_smoke.log
tail -2 gpurun_out/${R}_pytest_gpu.log; tail -2 gpurun_out/${R}_smoke.log
NO_PYTEST=1 ROUND=$R bash tools/gpu_round.sh
timeout -s KILL 600 python tools/fig2.py --size 2048 --widths 3,7,11,15,17 --md gpurun_out/${R}_fig2.md > gpurun_out/${R}_fig2_2048.json 2> gpurun_out/${R}_fig2_2048.err
timeout -s KILL 600 python tools/fig2.py --size 3520 --md gpurun_out/${R}_fig2.md > gpurun_out/${R}_fig2_3520.json 2> gpurun_out/${R}_fig2_3520.err
timeout -s KILL 900 ncu --metrics gpu__time_duration.sum --clock-control none --nvtx --nvtx-include "sepconv_timed/" \
   --csv --log-file gpurun_out/${R}_launches.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline \
   > gpurun_out/${R}_launches_bench.json 2> gpurun_out/${R}_launches_bench.err
echo "launch list rc=$?"
for spec in 5:sep-fused-tma1 17:sep-fused-tma2; do
  K=${spec%%:*}; C=${spec#*:}
  timeout -s KILL 900 ncu --set full --clock-control none --import-source on -k regex:stream_kernel -s 1 -c 1 \
    -o gpurun_out/${R}_${C}_k${K} python tools/prof_one.py --k $K --cand $C --n 1 > gpurun_out/${R}_prof_${C}_k${K}.log 2>&1
  echo "full $spec rc=$?"
done
python tools/ncu_summary.py gpurun_out/${R}_*.ncu-rep --out gpurun_out/${R}_ncu_summary.md > gpurun_out/${R}_ncu_summary.log 2>&1
rm -f gpurun_out/${R}_*.ncu-rep
ls gpurun_out | head -80
