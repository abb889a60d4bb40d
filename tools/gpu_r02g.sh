set -x
timeout 1800 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/r02g_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02g_pytest.log
timeout 600 python tools/sweep.py --workload c4_u64_2p30 flags=16 k=256,flags=16 k=256,flags=272 k=256,flags=272,M=32768 > gpurun_out/r02g_cluster_2p30.log 2>&1
timeout 600 python tools/sweep.py --workload c4_u64_2p28 flags=16 k=4096,tile=65536,flags=272,k_policy=fixed > gpurun_out/r02g_cluster_2p28.log 2>&1
