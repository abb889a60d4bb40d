set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "lookup or partition_level or sort_distributions or ablation_variants or bench_config_parity or edge_sizes" > gpurun_out/r02u_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02u_pytest.log
tail -3 gpurun_out/r02u_pytest.log
timeout 600 python tools/sweep.py --workload c4_u64_2p28 k=256 k=256,flags=512 k=256 k=256,flags=512 > gpurun_out/r02u_ab_c4.log 2>&1
timeout 600 python tools/sweep.py --workload c2_u32_2p27 k=256 k=256,flags=512 > gpurun_out/r02u_ab_c2.log 2>&1
for d in gaussian and4 staggered sorted dd; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c4_u64_2p28 k=256 k=256,flags=512 >> gpurun_out/r02u_ab_dists.log 2>&1; done
bash tools/ncu_one.sh r02u k_classify 1
