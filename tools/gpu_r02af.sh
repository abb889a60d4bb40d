timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or lookup" > gpurun_out/r02af_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02af_pytest.log
timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none pf0 pf2 pf6 /tmp/none > gpurun_out/r02af_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c2_u32_2p27 k=256 /tmp/none pf0 pf2 pf6 >> gpurun_out/r02af_ab.log 2>&1
