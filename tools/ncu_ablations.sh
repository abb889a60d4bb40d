#!/bin/bash
# ncu counters of the ablation variants: one full capture of the affected kernel per variant on
# 2^28 uniform u64 keys.  usage: tools/ncu_ablations.sh <tag>
TAG=${1:-abl}
run() {   # name kernel-regex skip one_sort-args...
  N=$1; K=$2; S=$3; shift 3
  timeout 900 ncu --set full --clock-control none -k regex:$K -s $S -c 1 -o gpurun_out/abl_${TAG}_${N} -f \
     python tools/one_sort.py --workload c4_u64_2p28 --warmup 0 --steps 1 "$@" > gpurun_out/abl_${TAG}_${N}.log 2>&1
  echo "$N rc=$?"
}
run cls8 k_classify 1
run cls1 k_classify 1 --cls_arrays 1
run recompute k_scatter 1 --flags 1
run scatter_bulk k_scatter 1
run scatter_regs k_scatter 1 --flags 32
run scatter_direct k_scatter 1 --flags 8
run small_oem k_small_block 4
run small_bitonic k_small_block 4 --flags 128
python tools/summarize_ablations.py $TAG > gpurun_out/abl_${TAG}_summarize.log 2>&1
rm -f gpurun_out/abl_${TAG}_*.ncu-rep     # gpurun_out/ comes back only under 64 MiB
