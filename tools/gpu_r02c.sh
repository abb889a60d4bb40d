set -x
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/r02c_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02c_pytest.log
timeout 900 compute-sanitizer --tool racecheck --kernel-name regex=k_ --print-limit 20 python tools/sanitize_run.py > gpurun_out/r02c_san_racecheck.log 2>&1
timeout 900 compute-sanitizer --tool memcheck --kernel-name regex=k_ --print-limit 20 python tools/sanitize_run.py > gpurun_out/r02c_san_memcheck.log 2>&1
for wl in c4_u64_2p28 c3_kv64_2p27 c2_u32_2p27 c3_kv32_2p27; do
  timeout 300 python tools/sweep.py --workload $wl flags=16 flags=48 > gpurun_out/r02c_ab_$wl.log 2>&1
done
bash tools/ncu_one.sh r02c k_scatter_bulk 0 c4_u64_2p28
