#!/bin/bash
# deeper rings for short segments (mid sizes), the carveout floor probe, BS grid crossover
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out /tmp/x
F="-std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -lineinfo -Ipaper_conf_asplos_phothilimthanaara13_b200/csrc"
nvcc $F tools/explore_mid.cu -o /tmp/x/explore_mid -lcuda &
nvcc $F tools/smem_floor.cu -o /tmp/x/smem_floor &
nvcc $F tools/bs_small.cu -o /tmp/x/bs_small &
wait
timeout -s KILL 300 /tmp/x/smem_floor > gpurun_out/r02e_smem_floor.txt 2>&1
EXPLORE_DEEP=1 timeout -s KILL 900 /tmp/x/explore_mid 2048 3520 4096 16384 > gpurun_out/r02e_deep.txt 2>&1
timeout -s KILL 300 /tmp/x/bs_small 500000 4194304 8388608 16777216 67108864 > gpurun_out/r02e_bs_small.txt 2>&1
cat gpurun_out/r02e_smem_floor.txt gpurun_out/r02e_deep.txt gpurun_out/r02e_bs_small.txt
