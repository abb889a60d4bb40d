set -x
for wl in c4_u64_2p28 c2_u32_2p27 c3_kv64_2p27 c3_kv32_2p27; do
  timeout 400 python tools/sweep.py --workload $wl flags=16 flags=268435472 > gpurun_out/r02j_ab_$wl.log 2>&1
done
timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "bench_config_parity or sort_distributions or edge_sizes or single_bucket" > gpurun_out/r02j_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02j_pytest.log
