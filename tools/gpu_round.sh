#!/bin/bash
# One GPU session: bench line, launch list and a full ncu capture of the top kernels.
# usage: tools/gpu_round.sh <tag> [workload]
set -x
TAG=${1:-r01}
WL=${2:-c4_u64_2p28}
mkdir -p gpurun_out
timeout 600 python bench.py --workload $WL > gpurun_out/bench_${TAG}_${WL}.json 2> gpurun_out/bench_${TAG}_${WL}.err
tail -c 3000 gpurun_out/bench_${TAG}_${WL}.json
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
