#!/bin/bash
# Round profile: launch list (one sort, gpu__time_duration + dram bytes) and full ncu captures of the
# three hot kernels of the default workload.  usage: tools/profile_round.sh <tag> [workload]
TAG=${1:-r01}
WL=${2:-c4_u64_2p28}
mkdir -p gpurun_out
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
echo "launches rc=$?"
# name:regex:skip -- skip picks the launch (k_small_block: classes are launched largest first; 4 = the 10-warp class)
for spec in "k_classify:k_classify:1" "k_scatter:k_scatter:1" "k_small:k_small_block:4"; do
  N=$(echo $spec | cut -d: -f1); K=$(echo $spec | cut -d: -f2); S=$(echo $spec | cut -d: -f3)
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
     -o gpurun_out/prof_${TAG}_${N} -f python tools/one_sort.py --workload $WL --warmup 0 --steps 1 \
     > gpurun_out/prof_${TAG}_${N}.log 2>&1
  echo "$N rc=$?"
done
# (the profiled libgss.so stays on the box: gpurun_out/ must stay under 64 MiB; rebuild the commit to map SASS lines)
python tools/summarize_profiles.py $TAG $WL paper_conf_ipps_leischneros10_b200/libgss.so gpurun_out > gpurun_out/summarize_${TAG}.log 2>&1
echo "summary rc=$?"
