set -x
timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "lookup or partition_level or sort_distributions or ablation_variants" > gpurun_out/r02v_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02v_pytest.log
tail -3 gpurun_out/r02v_pytest.log
for d in uniform and4 and3 gaussian; do GSS_DIST=$d timeout 300 bash tools/ab_run.sh c4_u64_2p28 k=256 /tmp/none clsu16 clsminb3 >> gpurun_out/r02v_ab.log 2>&1; done
GSS_DIST=uniform timeout 300 bash tools/ab_run.sh c2_u32_2p27 k=256 /tmp/none clsu16 clsminb3 >> gpurun_out/r02v_ab.log 2>&1
