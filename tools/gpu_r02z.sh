set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or single_bucket or bucket_sorter or edge_sizes or cluster" > gpurun_out/r02z_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02z_pytest.log
tail -3 gpurun_out/r02z_pytest.log
timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none nogrp unroll1 /tmp/none > gpurun_out/r02z_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c2_u32_2p27 k=256 /tmp/none nogrp unroll1 >> gpurun_out/r02z_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c3_kv64_2p27 k=256 /tmp/none nogrp unroll1 >> gpurun_out/r02z_ab.log 2>&1
