#!/bin/bash
# Full ncu capture of one kernel.  usage: tools/ncu_one.sh <tag> <kernel regex> <skip> [workload]
TAG=$1; K=$2; S=${3:-0}; WL=${4:-c4_u64_2p28}
timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
   -o gpurun_out/prof_${TAG}_${K} -f python tools/one_sort.py --workload $WL --warmup 0 --steps 1 \
   > gpurun_out/prof_${TAG}_${K}.log 2>&1
echo "$K rc=$?"
