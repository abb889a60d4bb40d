set -x
timeout 600 python bench.py > gpurun_out/r02k_bench.json 2> gpurun_out/r02k_bench.err
bash tools/profile_round.sh r02k c4_u64_2p28
for tool in memcheck racecheck synccheck; do
  timeout 900 compute-sanitizer --tool $tool --kernel-name regex=k_ --print-limit 20 python tools/sanitize_run.py > gpurun_out/r02k_san_$tool.log 2>&1
  echo "rc=$?" >> gpurun_out/r02k_san_$tool.log
done
du -sh gpurun_out
