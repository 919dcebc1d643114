#!/bin/bash
# store path 2 as a tuner candidate: the GPU suite, the mid-size legs, the headline
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
timeout -s KILL 1500 python -m pytest tests -x -q -m gpu -p no:cacheprovider > gpurun_out/${R:-r02v2}_pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/${R:-r02v2}_pytest_gpu.log
tail -2 gpurun_out/${R:-r02v2}_pytest_gpu.log
B="timeout -s KILL 900 python bench.py --no-cpu-baseline --no-e2e"
$B --steps 50 --warmup 3 --size 2048 --widths 3,7,11,15,17 > gpurun_out/${R:-r02v2}_bench_c2.json 2>/dev/null
$B --steps 50 --warmup 3 --size 3520 > gpurun_out/${R:-r02v2}_bench_c2p.json 2>/dev/null
$B --steps 50 --warmup 3 --size 4096 --widths 17 > gpurun_out/${R:-r02v2}_bench_c3.json 2>/dev/null
$B --steps 20 --warmup 5 > gpurun_out/${R:-r02v2}_bench_c4.json 2>/dev/null
$B --steps 20 --warmup 5 > gpurun_out/${R:-r02v2}_bench_c4_b.json 2>/dev/null
python tools/bench_summary.py gpurun_out/${R:-r02v2}_bench_*.json
