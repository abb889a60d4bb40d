timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions" > gpurun_out/r02ak_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ak_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27; do
  timeout 600 python tools/sweep.py --workload $wl k=0 k=0,flags=67108864 k=0 k=0,flags=67108864 >> gpurun_out/r02ak_ab.log 2>&1
done
for d in sorted dd and4; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c4_u64_2p28 k=0 k=0,flags=67108864 >> gpurun_out/r02ak_ab.log 2>&1; done
