#!/bin/bash
# ncu evidence: the launch list of a short bench and full captures of the fused kernel.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r01}
timeout -s KILL 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv \
   --log-file gpurun_out/${R}_launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline \
   --tune-reps 2 > gpurun_out/${R}_launches_bench.log 2>&1
for K in ${PROF_KS:-17 3 9}; do
  timeout -s KILL 900 ncu --set full --clock-control none --import-source on -k regex:stream_kernel -s 1 -c 1 \
    -o gpurun_out/${R}_sep_k${K} python tools/prof_one.py --k $K --n 1 > gpurun_out/${R}_prof_k${K}.log 2>&1
done
ls -la gpurun_out
