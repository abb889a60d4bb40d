#!/bin/bash
# Round profile: launch list (one sort, gpu__time_duration + dram bytes) and full ncu captures of the
# three hot kernels of the default workload.  usage: tools/profile_round.sh <tag> [workload]
TAG=${1:-r01}
WL=${2:-c4_u64_2p28}
mkdir -p gpurun_out
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
   --log-file gpurun_out/launches_${TAG}_${WL}.csv python tools/one_sort.py --workload $WL --warmup 1 --steps 1 > gpurun_out/launches_${TAG}.log 2>&1
echo "launches rc=$?"
for spec in "k_classify:0" "k_scatter:0" "k_small:1"; do
  K=${spec%%:*}; S=${spec##*:}
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
     -o gpurun_out/prof_${TAG}_${K} -f python tools/one_sort.py --workload $WL --warmup 0 --steps 1 \
     > gpurun_out/prof_${TAG}_${K}.log 2>&1
  echo "$K rc=$?"
done
python tools/summarize_profiles.py $TAG $WL paper_conf_ipps_leischneros10_b200/libgss.so gpurun_out > gpurun_out/summarize_${TAG}.log 2>&1
echo "summary rc=$?"
# keep the merged-back directory under the 64 MiB limit: drop the raw reports except the small-sort one
rm -f gpurun_out/prof_${TAG}_k_classify.ncu-rep gpurun_out/prof_${TAG}_k_scatter.ncu-rep
