timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "k_values or sort_distributions or full_size or bench_config" > gpurun_out/r02ag_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ag_pytest.log
timeout 900 python tools/sweep.py --workload c4_u64_2p30 k=512 k=512,flags=134217728 k=256 > gpurun_out/r02ag_sweep.log 2>&1
timeout 900 python tools/sweep.py --workload c4_u64_2p28 k=512 k=256 >> gpurun_out/r02ag_sweep.log 2>&1
timeout 900 python tools/sweep.py --workload c4_u64_2p29 k=512 k=256 >> gpurun_out/r02ag_sweep.log 2>&1
