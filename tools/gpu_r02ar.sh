timeout 1500 python -m pytest tests -m gpu -x -q -p no:cacheprovider > gpurun_out/r02ar_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ar_pytest.log
for wl in c4_u64_2p28 c2_u32_2p27 c3_kv64_2p27 c3_kv32_2p27; do
  timeout 600 python tools/sweep.py --workload $wl k=0 k=0 >> gpurun_out/r02ar_ab.log 2>&1
done
for d in sorted dd and4; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c4_u64_2p28 k=0 >> gpurun_out/r02ar_ab.log 2>&1; done
timeout 600 python tools/sweep.py --workload c4_u64_2p30 k=0 >> gpurun_out/r02ar_ab.log 2>&1
