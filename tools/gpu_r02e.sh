set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "descending or gss_hpp" > gpurun_out/r02e_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02e_pytest.log
for wl in c5_kv64_2p29 c3_kv64_2p27; do
  timeout 400 python tools/sweep.py --workload $wl flags=16 flags=48 > gpurun_out/r02e_ab_$wl.log 2>&1
done
bash tools/ncu_one.sh r02e k_small_block 4 c4_u64_2p28
bash tools/ncu_one.sh r02e k_classify 0 c4_u64_2p28
