timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or edge_sizes or bench_config_parity or lookup" > gpurun_out/r02ab_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ab_pytest.log
timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none io1 io3 /tmp/none > gpurun_out/r02ab_ab.log 2>&1
GSS_DIST=sorted timeout 600 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none io1 io3 >> gpurun_out/r02ab_ab.log 2>&1
timeout 600 bash tools/ab_run.sh c4_u64_2p29 k=256 /tmp/none io1 >> gpurun_out/r02ab_ab.log 2>&1
