#!/bin/bash
# usage: tools/ncu_cfg.sh <tag> <kernel regex> <skip> "<one_sort args>"
TAG=$1; K=$2; S=${3:-0}; A=$4
timeout 900 ncu --set full --clock-control none --import-source on -k regex:$K -s $S -c 1 \
   -o gpurun_out/prof_${TAG}_${K} -f python tools/one_sort.py --warmup 0 --steps 1 $A > gpurun_out/prof_${TAG}_${K}.log 2>&1
echo "$K rc=$?"
