timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r02as_smoke.log 2>&1
timeout 600 python bench.py --no-cpu-baseline > gpurun_out/r02as_bench.json 2>/dev/null
