cd $GRAFT_REPO_ROOT
ncu --set full --clock-control none --import-source on -k regex:stream_kernel -s 1 -c 1 -o gpurun_out/r01_k13_sm1 ./tools/explore 10 13 > gpurun_out/r01_k13_sm1.log 2>&1
ncu --set full --clock-control none --import-source on -k regex:stream_kernel -s 13 -c 1 -o gpurun_out/r01_k13_sm2 ./tools/explore 10 13 > gpurun_out/r01_k13_sm2.log 2>&1
ls gpurun_out
