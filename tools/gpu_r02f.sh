set -x
timeout 1200 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "descending or gss_hpp or ablation_variants or bench_config_parity or edge_sizes" > gpurun_out/r02f_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02f_pytest.log
timeout 400 python tools/sweep.py --workload c4_u64_2p28 flags=16 flags=144 cls_arrays=1,flags=16 cls_arrays=2,flags=16 > gpurun_out/r02f_ab_c4.log 2>&1
