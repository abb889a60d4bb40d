#!/bin/bash
# quick tests + bench + launch list (+ optional one ncu capture).  usage: tools/gpu_quick.sh <tag> [workload] [pytest -k] [ncu kernel] [skip]
TAG=${1:-rx}
WL=${2:-c4_u64_2p28}
K=${3:-"partition or (sort_distributions and uniform) or edge or overflow"}
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider -k "$K" > gpurun_out/gpu_tests_${TAG}.log 2>&1
echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests_${TAG}.log
timeout 600 python bench.py --workload $WL --no-cpu-baseline > gpurun_out/bench_${TAG}_${WL}.json 2> gpurun_out/bench_${TAG}_${WL}.err
echo "bench rc=$?"
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
cp paper_conf_ipps_leischneros10_b200/libgss.so gpurun_out/libgss_${TAG}.so
if [ -n "$4" ]; then tools/ncu_one.sh $TAG $4 ${5:-0} $WL; fi
