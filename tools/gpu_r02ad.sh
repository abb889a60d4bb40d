timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or single_bucket or bucket_sorter or edge_sizes or c1_config or float" > gpurun_out/r02ad_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ad_pytest.log
timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none nodirect /tmp/none > gpurun_out/r02ad_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c2_u32_2p27 k=256 /tmp/none nodirect >> gpurun_out/r02ad_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c3_kv64_2p27 k=256 /tmp/none nodirect >> gpurun_out/r02ad_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c3_kv32_2p27 k=256 /tmp/none nodirect >> gpurun_out/r02ad_ab.log 2>&1
