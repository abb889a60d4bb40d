set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "distributed or partition_by_eq or capacity" > gpurun_out/r02b_pytest_dist.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02b_pytest_dist.log
for tool in memcheck racecheck synccheck; do
  timeout 900 compute-sanitizer --tool $tool --kernel-name regex=k_ --print-limit 20 python tools/sanitize_run.py > gpurun_out/r02b_san_$tool.log 2>&1
  echo "rc=$?" >> gpurun_out/r02b_san_$tool.log
done
timeout 600 python bench.py --force-dist --no-cpu-baseline > gpurun_out/r02b_bench_dist1.json 2> gpurun_out/r02b_bench_dist1.err
timeout 600 python bench.py --force-dist --workload c5_kv64_2p29 > gpurun_out/r02b_bench_dist1_c5.json 2> gpurun_out/r02b_bench_dist1_c5.err
