cd "${GRAFT_REPO_ROOT}"
mkdir -p gpurun_out
timeout -s KILL 600 python -m pytest tests/test_gpu_bs.py tests/test_gpu_fuzz.py -m gpu -q -x -p no:cacheprovider > gpurun_out/r02f_pytest_bs.log 2>&1; echo "rc=$?" >> gpurun_out/r02f_pytest_bs.log
B="timeout -s KILL 600 python bench.py"
$B --steps 20 --warmup 3 --workload blackscholes --options 500000 > gpurun_out/r02f_bench_bs_500k.json 2> gpurun_out/r02f_bench_bs_500k.err
$B --steps 10 --warmup 3 --workload blackscholes > gpurun_out/r02f_bench_bs.json 2> gpurun_out/r02f_bench_bs.err
python tools/bench_summary.py gpurun_out/r02f_bench_*.json
tail -3 gpurun_out/r02f_pytest_bs.log
