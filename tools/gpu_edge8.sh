#!/bin/bash
# the 8-byte store paths on even-width right edges: sanitizer, the GPU suite, bench A/B material
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
SANITIZE_KS=3,7,15,17 ROUND=r02v SAN_TIMEOUT=900 bash tools/gpu_sanitize.sh
timeout -s KILL 1500 python -m pytest tests -x -q -m gpu -p no:cacheprovider > gpurun_out/r02v_pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/r02v_pytest_gpu.log
tail -2 gpurun_out/r02v_pytest_gpu.log
B="timeout -s KILL 900 python bench.py --no-cpu-baseline --no-e2e"
$B --steps 20 --warmup 5 > gpurun_out/r02v_bench_c4_a.json 2>/dev/null
$B --steps 20 --warmup 5 > gpurun_out/r02v_bench_c4_b.json 2>/dev/null
$B --steps 50 --warmup 3 --size 2048 --widths 3,7,11,15,17 > gpurun_out/r02v_bench_c2.json 2>/dev/null
$B --steps 50 --warmup 3 --size 3520 > gpurun_out/r02v_bench_c2p.json 2>/dev/null
python tools/bench_summary.py gpurun_out/r02v_bench_*.json
K17_PROBE_K=15 timeout -s KILL 600 python tools/k17_probe.py > gpurun_out/r02v_k15_probe.txt 2>&1; head -4 gpurun_out/r02v_k15_probe.txt
