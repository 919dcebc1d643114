cd "${GRAFT_REPO_ROOT}"
mkdir -p gpurun_out
for spec in 17:sep-fused-tma4 17:sep-fused-tma2; do
  K=${spec%%:*}; C=${spec#*:}
  timeout -s KILL 600 ncu --section SourceCounters --import-source on --clock-control none \
     -k regex:stream_kernel -s 1 -c 1 -o /tmp/bank16_$C python tools/prof_one.py --k $K --cand $C --n 1 --size 16384 > gpurun_out/r02k_bank16_$C.log 2>&1
  ncu -i /tmp/bank16_$C.ncu-rep --page source --csv --print-source sass > gpurun_out/r02k_bank16_src_$C.csv 2>>gpurun_out/r02k_bank16_$C.log
done
