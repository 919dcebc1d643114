#!/bin/bash
# SOR graph replay: GPU tests, the graph probe, the Poisson bench legs (with and without graphs)
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
timeout -s KILL 600 python -m pytest tests/test_gpu_sor.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r02j_pytest_sor.log 2>&1; echo "rc=$?" >> gpurun_out/r02j_pytest_sor.log
tail -3 gpurun_out/r02j_pytest_sor.log
B="timeout -s KILL 600 python bench.py"
$B --steps 10 --warmup 3 --workload poisson --size 2048 > gpurun_out/r02j_bench_poisson_2048.json 2> gpurun_out/r02j_bench_poisson_2048.err
SOR_GRAPHS=0 $B --steps 10 --warmup 3 --workload poisson --size 2048 > gpurun_out/r02j_bench_poisson_2048_nograph.json 2> /dev/null
$B --steps 5 --warmup 3 --workload poisson --size 16384 > gpurun_out/r02j_bench_poisson_16384.json 2> gpurun_out/r02j_bench_poisson_16384.err
python tools/bench_summary.py gpurun_out/r02j_bench_*.json
