#!/bin/bash
# One GPU session: smoke, the -m gpu suite, a short bench.  Logs to gpurun_out/.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,memory.used --format=csv > gpurun_out/nvsmi.txt 2>&1
timeout -s KILL 120 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/smoke.log
tail -3 gpurun_out/smoke.log
if [ -n "$SANITIZE" ]; then
  timeout -s KILL 300 compute-sanitizer --tool memcheck python tools/sanitize.py ${SANITIZE_KS:-3} > gpurun_out/sanitize.log 2>&1; tail -5 gpurun_out/sanitize.log
fi
if [ -z "$NO_PYTEST" ]; then
  timeout -s KILL ${PYTEST_TIMEOUT:-900} python -m pytest tests -m gpu -q -x --timeout=300 ${PYTEST_ARGS} > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
  tail -15 gpurun_out/pytest_gpu.log
fi
if [ -z "$NO_BENCH" ]; then
  timeout -s KILL 400 python bench.py ${BENCH_ARGS:---steps 5 --warmup 3} > gpurun_out/bench.log 2>gpurun_out/bench.err; echo "bench rc=$?" >> gpurun_out/bench.err
  cat gpurun_out/bench.log; tail -5 gpurun_out/bench.err
fi
