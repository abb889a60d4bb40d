timeout 300 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none nowrite > gpurun_out/r02w_ab.log 2>&1
