timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "graph or bench_config or sort_distributions" > gpurun_out/r02aq_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02aq_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27 c1_u32_2p16; do
  timeout 600 python tools/sweep.py --workload $wl k=0,flags=16 k=0,flags=16777232 k=0,flags=16 k=0,flags=16777232 >> gpurun_out/r02aq_ab.log 2>&1
done
timeout 300 python bench.py --workload c1_u32_2p16 --no-cpu-baseline > gpurun_out/r02aq_bench_c1.json 2>/dev/null
