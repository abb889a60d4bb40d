#!/bin/bash
# Full ncu captures of the given kernels (regex:skip pairs), summarised into gpurun_out/<tag>_ncu_summary.md;
# raw reports are deleted so the merged-back directory stays small.
# usage: tools/ncu_pair.sh <tag> <workload> <kernel:skip> [<kernel:skip> ...]
TAG=$1; WL=$2; shift 2
mkdir -p gpurun_out
for spec in "$@"; do
  K=${spec%%:*}; S=${spec##*:}
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
     -o gpurun_out/prof_${TAG}_${K} -f python tools/one_sort.py --workload $WL --warmup 0 --steps 1 \
     > gpurun_out/prof_${TAG}_${K}.log 2>&1
  echo "$K rc=$?"
done
python tools/summarize_profiles.py $TAG $WL paper_conf_ipps_leischneros10_b200/libgss.so gpurun_out > gpurun_out/sum_${TAG}.log 2>&1
echo "summary rc=$?"

rm -f gpurun_out/*.ncu-rep
