timeout 1500 python -m pytest tests -m gpu -x -q -p no:cacheprovider > gpurun_out/r02aj_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02aj_pytest.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r02aj_smoke.log 2>&1
echo "smoke rc=$?" >> gpurun_out/r02aj_smoke.log
