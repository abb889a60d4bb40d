set -x
for d in uniform sorted dd; do
  GSS_DIST=$d timeout 900 bash tools/ab_run.sh c2_u32_2p27 "flags=16" ur2 noru > gpurun_out/r02q_ab_c2_$d.log 2>&1
  GSS_DIST=$d timeout 900 bash tools/ab_run.sh c4_u64_2p28 "flags=16" ur2 noru > gpurun_out/r02q_ab_c4_$d.log 2>&1
done
