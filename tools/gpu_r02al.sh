timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=0 /tmp/none lutonly3 lutonly2 > gpurun_out/r02al_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c2_u32_2p27 k=0 /tmp/none lutonly3 lutonly2 >> gpurun_out/r02al_ab.log 2>&1
GSS_DIST=gaussian timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=0 /tmp/none lutonly3 >> gpurun_out/r02al_ab.log 2>&1
