timeout 1500 python -m pytest tests -m gpu -x -q -p no:cacheprovider > gpurun_out/r02ap_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ap_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27 c1_u32_2p16 c3_kv64_2p27; do
  timeout 600 python tools/sweep.py --workload $wl k=0,flags=16 k=0,flags=16777232 k=0,flags=16 k=0,flags=16777232 >> gpurun_out/r02ap_ab.log 2>&1
done
