#!/bin/bash
# Round evidence in one GPU session: tests, smoke, default bench, batch bench, ncu launch list
# and full captures of the tuned fused kernels.  Logs to gpurun_out/.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r01}
NO_BENCH=1 bash tools/gpu_check.sh
timeout -s KILL 500 python bench.py --steps 10 --warmup 3 > gpurun_out/${R}_bench.json 2> gpurun_out/${R}_bench.err; echo "bench rc=$?"
timeout -s KILL 500 python bench.py --workload batch --steps 5 --warmup 3 --no-cpu-baseline > gpurun_out/${R}_bench_batch.json 2> gpurun_out/${R}_bench_batch.err; echo "batch rc=$?"
cat gpurun_out/${R}_bench.json gpurun_out/${R}_bench_batch.json | cut -c1-400
PROF="${PROF:-17:sep-fused-tma3 9:sep-fused-tma0 3:sep-fused-tma2}" bash tools/gpu_profile.sh > /dev/null 2>&1
ls gpurun_out
