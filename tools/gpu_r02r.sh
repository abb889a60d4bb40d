set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -q -p no:cacheprovider -k "fused_scatter_segments or virtual_ranks" > gpurun_out/r02r_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02r_pytest.log
timeout 900 bash tools/ab_run.sh c4_u64_2p28 flags=16 oneload base > gpurun_out/r02r_ab_c4.log 2>&1
