#!/bin/bash
# On the GPU box: time every variants/libgss_*.so on a workload with tools/sweep.py.
# usage: tools/ab_run.sh <workload> <cfg> [names...]
WL=$1; CFG=$2; shift 2
cp paper_conf_ipps_leischneros10_b200/libgss.so /tmp/libgss_default.so
for so in ${@:-variants/libgss_*.so}; do
  [ "$so" = /tmp/none ] && so=/tmp/libgss_default.so
  [ -f "$so" ] || so=variants/libgss_$so.so
  cp $so paper_conf_ipps_leischneros10_b200/libgss.so
  echo "== $so"; python tools/sweep.py --workload $WL $CFG
done
cp /tmp/libgss_default.so paper_conf_ipps_leischneros10_b200/libgss.so
