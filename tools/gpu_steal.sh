#!/bin/bash
# Work stealing between warps (R27): parity, compute-sanitizer over the stealing paths,
# burst and sustained timings, the tuner's own timings, and bench.py with stealing seeded.
# Evidence: profiles/r02_steal_sched.txt, profiles/r02_sanitize_steal_*.log.
mkdir -p gpurun_out
timeout -s KILL 600 python -m pytest tests/test_gpu_parity.py -x -q -k "stealing or mutated or repeated or tuner" \
    > gpurun_out/steal_pytest.log 2>&1; echo "pytest rc=$?"; tail -n 3 gpurun_out/steal_pytest.log
for tool in memcheck racecheck synccheck; do
  timeout -s KILL 900 compute-sanitizer --tool $tool --error-exitcode 9 python tools/sanitize.py \
      > gpurun_out/steal_san_$tool.log 2>&1; echo "$tool rc=$?"; tail -n 2 gpurun_out/steal_san_$tool.log
done
{
timeout -s KILL 300 python tools/sched_check.py --size 16384 --k 17 --cands tma4,tma2 --scheds 0:0,9:0:4,9:0:2,9:0:8,18:0:4,18:0,27:0:4
timeout -s KILL 300 python tools/steal_ab.py --size 16384 --k 17 --choices tma3,tma4@9:0:4,tma2@9:0:4,tma4@18:0:4,tma2@18:0:4,tma4@18:0:0
timeout -s KILL 300 python tools/steal_ab.py --size 16384 --k 13 --choices tma0s8,tma2@9:0:4,tma4@9:0:4,tma2@18:0:4
timeout -s KILL 300 python tools/sched_check.py --size 4096 --k 17 --cands tma2,tma4,tma5 --n 40 --scheds 0:0,37:0:4,37:0:2,74:0:4
timeout -s KILL 300 python tools/sched_check.py --size 2048 --k 17 --cands tma2,tma4 --n 40 --scheds 0:0,74:0:4,74:0:2,148:0:4
SEPCONV_TUNE_LOG=gpurun_out/tune_steal.log timeout -s KILL 600 python tools/sched_check.py --size 16384 --k 17 \
    --cands tma4,tma3 --scheds 0:0,9:148:4,9:148:0,18:148:4,18:148:0 --tune --retime
grep "st[1-9]\|accepted" gpurun_out/tune_steal.log
} 2>&1 | tee gpurun_out/steal_sched.txt
for r in 1 2; do
  SEPCONV_TUNE_LOG=gpurun_out/tune_bench_$r.log timeout -s KILL 900 python bench.py --no-cpu-baseline \
      > gpurun_out/bench_steal_$r.json 2> gpurun_out/bench_steal_$r.err
  python tools/bench_summary.py gpurun_out/bench_steal_$r.json
  grep "st[1-9]" gpurun_out/tune_bench_$r.log | grep "k1[357]"
done
