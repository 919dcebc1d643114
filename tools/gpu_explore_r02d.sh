#!/bin/bash
# round-2 follow-up explorations: dry-pass instruction warm-up of the fused kernel at mid sizes,
# the shared-memory carveout floor, Black-Scholes grid variants at the paper's 500 000 options
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out /tmp/x
F="-std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -lineinfo -Ipaper_conf_asplos_phothilimthanaara13_b200/csrc"
nvcc $F tools/explore_mid.cu -o /tmp/x/explore_mid -lcuda &
nvcc $F tools/smem_floor.cu -o /tmp/x/smem_floor &
nvcc $F tools/bs_small.cu -o /tmp/x/bs_small &
wait
timeout -s KILL 300 /tmp/x/smem_floor > gpurun_out/r02d_smem_floor.txt 2>&1
timeout -s KILL 300 /tmp/x/bs_small > gpurun_out/r02d_bs_small.txt 2>&1
EXPLORE_IWARM=1 timeout -s KILL 900 /tmp/x/explore_mid 2048 4096 3520 > gpurun_out/r02d_iwarm.txt 2>&1
cat gpurun_out/r02d_smem_floor.txt gpurun_out/r02d_bs_small.txt gpurun_out/r02d_iwarm.txt
