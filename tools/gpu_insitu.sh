#!/bin/bash
# in-step refinement: new GPU tests, the default bench twice (with and without refinement)
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
timeout -s KILL 900 python -m pytest tests/test_gpu_bench_contract.py tests/test_gpu_parity.py -m gpu -q -x -p no:cacheprovider -k "set_choice or in_step or image_workload" > gpurun_out/r02m_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/r02m_pytest.log
tail -3 gpurun_out/r02m_pytest.log
B="timeout -s KILL 900 python bench.py"
$B --steps 10 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/r02m_bench_c4.json 2> gpurun_out/r02m_bench_c4.err
$B --steps 10 --warmup 3 --no-cpu-baseline --no-e2e --insitu-steps 0 > gpurun_out/r02m_bench_c4_noinsitu.json 2> /dev/null
$B --steps 10 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/r02m_bench_c4_b.json 2> gpurun_out/r02m_bench_c4_b.err
$B --steps 10 --warmup 3 --no-cpu-baseline --no-e2e --insitu-steps 0 > gpurun_out/r02m_bench_c4_noinsitu_b.json 2> /dev/null
python tools/bench_summary.py gpurun_out/r02m_bench_*.json
grep "in-step" gpurun_out/r02m_bench_c4*.err
