#!/bin/bash
# One evidence session: GPU tests, smoke, every bench leg (BASELINE configs C1-C5 + NEXT legs),
# per-call latency.  Logs to gpurun_out/ (R = round tag).
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
R=${ROUND:-r02}
if [ -z "$NO_PYTEST" ]; then
  timeout -s KILL 1500 python -m pytest tests -m gpu -q -x -p no:cacheprovider --timeout=600 > gpurun_out/${R}_pytest_gpu.log 2>&1
  echo "pytest rc=$?" >> gpurun_out/${R}_pytest_gpu.log; tail -3 gpurun_out/${R}_pytest_gpu.log
  timeout -s KILL 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${R}_smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/${R}_smoke.log
fi
B="timeout -s KILL 900 python bench.py"
$B --steps 10 --warmup 3 > gpurun_out/${R}_bench_c4.json 2> gpurun_out/${R}_bench_c4.err
$B --steps 20 --warmup 3 --size 64 --widths 3 > gpurun_out/${R}_bench_c1.json 2> gpurun_out/${R}_bench_c1.err
$B --steps 20 --warmup 3 --size 2048 --widths 3,7,11,15,17 > gpurun_out/${R}_bench_c2.json 2> gpurun_out/${R}_bench_c2.err
$B --steps 20 --warmup 3 --size 3520 --widths 3,5,7,9,11,13,15,17 --no-e2e > gpurun_out/${R}_bench_c2p.json 2> gpurun_out/${R}_bench_c2p.err
$B --steps 20 --warmup 3 --size 4096 --widths 17 > gpurun_out/${R}_bench_c3.json 2> gpurun_out/${R}_bench_c3.err
$B --steps 5 --warmup 3 --workload batch > gpurun_out/${R}_bench_c5.json 2> gpurun_out/${R}_bench_c5.err
$B --steps 10 --warmup 3 --workload poisson --size 2048 > gpurun_out/${R}_bench_poisson_2048.json 2> gpurun_out/${R}_bench_poisson_2048.err
$B --steps 5 --warmup 3 --workload poisson --size 16384 > gpurun_out/${R}_bench_poisson_16384.json 2> gpurun_out/${R}_bench_poisson_16384.err
$B --steps 20 --warmup 3 --workload blackscholes --options 500000 > gpurun_out/${R}_bench_bs_500k.json 2> gpurun_out/${R}_bench_bs_500k.err
$B --steps 10 --warmup 3 --workload blackscholes > gpurun_out/${R}_bench_bs.json 2> gpurun_out/${R}_bench_bs.err
AUTO_ONLY=1 timeout -s KILL 300 python tools/small_latency.py > gpurun_out/${R}_small_latency.txt 2>&1
python tools/bench_summary.py gpurun_out/${R}_bench_*.json
