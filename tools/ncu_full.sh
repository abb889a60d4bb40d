#!/bin/bash
# Full ncu captures of the three hot kernels of one sort.
# usage: tools/ncu_full.sh <tag> [workload]
TAG=${1:-r01}
WL=${2:-c4_u64_2p28}
mkdir -p gpurun_out
for spec in "k_small:1" "k_classify:0" "k_scatter:0"; do
  K=${spec%%:*}; S=${spec##*:}
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
     -o gpurun_out/prof_${TAG}_${K} -f python tools/one_sort.py --workload $WL --warmup 0 --steps 1 \
     > gpurun_out/prof_${TAG}_${K}.log 2>&1
  echo "$K rc=$?"
done
