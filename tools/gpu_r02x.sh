set -x
timeout 600 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions or edge_sizes or k_values or bench_config_parity or lookup or deterministic or graph_replay" > gpurun_out/r02x_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02x_pytest.log
tail -5 gpurun_out/r02x_pytest.log
timeout 600 python tools/sweep.py --workload c4_u64_2p28 k=256 k=256,flags=134217728 k=256 k=256,flags=134217728 > gpurun_out/r02x_ab.log 2>&1
for d in sorted dd and4; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c4_u64_2p28 k=256 k=256,flags=134217728 >> gpurun_out/r02x_ab.log 2>&1; done
timeout 300 python tools/sweep.py --workload c4_u64_2p29 k=256 k=256,flags=134217728 >> gpurun_out/r02x_ab.log 2>&1
