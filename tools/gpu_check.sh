#!/bin/bash
# tests + bench + launch list in one GPU session.  usage: tools/gpu_check.sh <tag> [workload] [pytest -k expr]
TAG=${1:-r01}
WL=${2:-c4_u64_2p28}
K=${3:-}
mkdir -p gpurun_out
if [ -n "$K" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider -k "$K" > gpurun_out/gpu_tests_${TAG}.log 2>&1
else
  timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider > gpurun_out/gpu_tests_${TAG}.log 2>&1
fi
echo "tests rc=$?"; tail -3 gpurun_out/gpu_tests_${TAG}.log
timeout 600 python bench.py --workload $WL > gpurun_out/bench_${TAG}_${WL}.json 2> gpurun_out/bench_${TAG}_${WL}.err
echo "bench rc=$?"
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
echo "ncu rc=$?"
