set -x
timeout 900 bash tools/ab_run.sh c4_u64_2p28 flags=16 spread nospread > gpurun_out/r02o_ab_c4.log 2>&1
timeout 900 bash tools/ab_run.sh c2_u32_2p27 flags=16 spread nospread > gpurun_out/r02o_ab_c2.log 2>&1
timeout 900 bash tools/ab_run.sh c3_kv64_2p27 flags=16 spread nospread > gpurun_out/r02o_ab_kv64.log 2>&1
