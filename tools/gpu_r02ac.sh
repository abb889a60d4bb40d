for t in memcheck racecheck synccheck; do
  timeout 1200 compute-sanitizer --tool $t --error-exitcode 9 python tools/sanitize_run.py > gpurun_out/r02ac_sanitize_$t.log 2>&1
  echo "$t rc=$?" >> gpurun_out/r02ac_sanitize_$t.log
  tail -2 gpurun_out/r02ac_sanitize_$t.log
done
