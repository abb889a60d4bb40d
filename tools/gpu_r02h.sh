set -x
timeout 900 bash tools/ab_run.sh c4_u64_2p28 flags=16 base pairload > gpurun_out/r02h_ab_c4.log 2>&1
timeout 900 bash tools/ab_run.sh c2_u32_2p27 flags=16 base pairload > gpurun_out/r02h_ab_c2.log 2>&1
timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "bench_config_parity or deterministic or full_size_elementwise" > gpurun_out/r02h_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02h_pytest.log
