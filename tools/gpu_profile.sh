#!/bin/bash
# ncu evidence: the launch list of a short bench and full captures of chosen kernels.
#   PROF="17:sep-fused-tma0 3:sep-fused-tma2" ROUND=r01 bash tools/gpu_profile.sh
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r01}
if [ -z "$NO_LAUNCHES" ]; then
# only the timed region of bench.py (NVTX range "sepconv_timed"), not the tuner's sweep
timeout -s KILL 900 ncu --metrics gpu__time_duration.sum --clock-control none --nvtx --nvtx-include "sepconv_timed/" \
   --csv --log-file gpurun_out/${R}_launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline \
   > gpurun_out/${R}_launches_bench.log 2>&1
fi
for spec in ${PROF:-17:sep-fused-tma0}; do
  K=${spec%%:*}; C=${spec#*:}
  timeout -s KILL 900 ncu --set full --clock-control none --import-source on -k regex:"stream_kernel|conv2d_kernel" -s 1 -c 1 \
    -o gpurun_out/${R}_${C}_k${K} python tools/prof_one.py --k $K --cand $C --n 1 > gpurun_out/${R}_prof_${C}_k${K}.log 2>&1
done
ls -la gpurun_out
# summarise on the box (reports are ~10 MB each; gpurun copies back at most 64 MiB)
if [ -n "$SUMMARIZE" ]; then
  python tools/ncu_summary.py gpurun_out/${R}_*.ncu-rep --out gpurun_out/${R}_ncu_summary.md --traffic gpurun_out/traffic.json > /dev/null 2>&1
  for f in gpurun_out/${R}_*.ncu-rep; do case "$f" in *${KEEP:-k17}.ncu-rep) ;; *) rm -f "$f";; esac; done
fi
ls -la gpurun_out
