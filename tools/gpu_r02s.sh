set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "virtual_ranks or sort_distributions or single_bucket or edge_sizes" > gpurun_out/r02s_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02s_pytest.log
timeout 900 bash tools/ab_run.sh c2_u32_2p27 flags=16 ol32 ol0 > gpurun_out/r02s_ab_c2.log 2>&1
timeout 900 bash tools/ab_run.sh c4_u64_2p28 flags=16 ol32 ol0 > gpurun_out/r02s_ab_c4.log 2>&1
