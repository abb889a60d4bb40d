timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or single_bucket or partition_level or edge_sizes" > gpurun_out/r02aa_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02aa_pytest.log
timeout 900 python tools/sweep.py --workload c4_u64_2p28 k=256 k=256,fill_div=2 k=256,fill_div=3 k=256,fill_div=6 k=256,fill_div=8 k=128 k=128,fill_div=8 k=512 k=256,M=8192 > gpurun_out/r02aa_sweep.log 2>&1
timeout 900 python tools/sweep.py --workload c4_u64_2p30 k=512 k=256 k=512,fill_div=2 k=512,fill_div=8 >> gpurun_out/r02aa_sweep.log 2>&1
