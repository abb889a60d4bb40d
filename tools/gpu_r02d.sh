set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "distributed or partition_by_eq or capacity or bench_config_parity" > gpurun_out/r02d_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02d_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27; do
  timeout 300 python tools/sweep.py --workload $wl flags=16 flags=48 > gpurun_out/r02d_ab_$wl.log 2>&1
done
timeout 600 python bench.py --force-dist --no-cpu-baseline --steps 5 > gpurun_out/r02d_bench_dist1.json 2> gpurun_out/r02d_bench_dist1.err
timeout 600 python bench.py --force-dist --no-cpu-baseline --steps 5 --workload c5_kv64_2p29 > gpurun_out/r02d_bench_dist1_c5.json 2> gpurun_out/r02d_bench_dist1_c5.err
timeout 600 python bench.py --force-dist --fused --no-cpu-baseline --steps 5 > gpurun_out/r02d_bench_dist1_fused.json 2> gpurun_out/r02d_bench_dist1_fused.err
