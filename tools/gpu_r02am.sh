timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or k_values or bench_config_parity or c1_config or edge_sizes" > gpurun_out/r02am_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02am_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27 c3_kv64_2p27 c4_u64_2p30; do
  timeout 600 python tools/sweep.py --workload $wl k=0 k=0,flags=33554432 k=0 k=0,flags=33554432 >> gpurun_out/r02am_ab.log 2>&1
done
