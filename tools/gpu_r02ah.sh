timeout 1200 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or edge_sizes or k_values or bench_config_parity or lookup or descending or float or c1_config or deterministic or full_size or host_pipeline or graph" > gpurun_out/r02ah_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ah_pytest.log
for wl in c2_u32_2p27 c3_kv64_2p27 c3_kv32_2p27 c5_kv64_2p29; do
  timeout 600 python tools/sweep.py --workload $wl k=0 k=0,flags=134217728 k=0 k=0,flags=134217728 >> gpurun_out/r02ah_ab.log 2>&1
done
for d in sorted dd and4; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c2_u32_2p27 k=0 k=0,flags=134217728 >> gpurun_out/r02ah_ab.log 2>&1; done
for d in sorted dd; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c3_kv64_2p27 k=0 k=0,flags=134217728 >> gpurun_out/r02ah_ab.log 2>&1; done
