set -x
timeout 900 bash tools/ab_run.sh c4_u64_2p28 flags=16 wb nowb > gpurun_out/r02l_ab_c4.log 2>&1
timeout 900 bash tools/ab_run.sh c2_u32_2p27 flags=16 wb nowb > gpurun_out/r02l_ab_c2.log 2>&1
timeout 1500 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -x -k "not distributed and not capacity" > gpurun_out/r02l_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02l_pytest.log
