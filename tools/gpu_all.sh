#!/bin/bash
# Full GPU test suite + default bench line + launch list.  usage: tools/gpu_all.sh <tag> [workload]
TAG=${1:-rx}
WL=${2:-c4_u64_2p28}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/smi_${TAG}.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q -p no:cacheprovider > gpurun_out/gpu_tests_${TAG}.log 2>&1
echo "tests rc=$?"; tail -3 gpurun_out/gpu_tests_${TAG}.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_${TAG}.log 2>&1; echo "smoke rc=$?"
timeout 600 python bench.py --workload $WL > gpurun_out/bench_${TAG}_${WL}.json 2> gpurun_out/bench_${TAG}_${WL}.err
echo "bench rc=$?"; cat gpurun_out/bench_${TAG}_${WL}.json | head -c 4000
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
echo "launches rc=$?"
