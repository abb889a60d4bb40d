#!/bin/bash
# Round-end evidence of the final tree (r02d): GPU tests, smoke, bench lines of every workload, one-rank
# distributed lines, the reference arm, launch list + ncu summaries.  (Distribution sweeps: r02c.)
set -x
TAG=r02d
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,driver_version --format=csv > gpurun_out/${TAG}_smi.txt
timeout 1800 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/${TAG}_pytest_gpu.log 2>&1
echo "pytest rc=$?" >> gpurun_out/${TAG}_pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${TAG}_smoke.log 2>&1
echo "smoke rc=$?" >> gpurun_out/${TAG}_smoke.log
timeout 600 python bench.py > gpurun_out/${TAG}_bench_c4_u64_2p28.json 2> gpurun_out/${TAG}_bench_c4_u64_2p28.err
for wl in c1_u32_2p16 c2_u32_2p27 c3_u64_2p27 c3_kv64_2p27 c3_kv32_2p27 c4_u64_2p29 c4_u64_2p30 c5_kv64_2p29; do
  timeout 600 python bench.py --workload $wl --no-cpu-baseline > gpurun_out/${TAG}_bench_$wl.json 2> gpurun_out/${TAG}_bench_$wl.err
done
timeout 600 python bench.py --force-dist --no-cpu-baseline --steps 5 > gpurun_out/${TAG}_bench_dist1_c4.json 2> gpurun_out/${TAG}_bench_dist1_c4.err
timeout 600 python bench.py --force-dist --fused --no-cpu-baseline --steps 5 > gpurun_out/${TAG}_bench_dist1_c4_fused.json 2> gpurun_out/${TAG}_bench_dist1_c4_fused.err
timeout 900 python bench.py --force-dist --no-cpu-baseline --steps 5 --workload c5_kv64_2p29 > gpurun_out/${TAG}_bench_dist1_c5.json 2> gpurun_out/${TAG}_bench_dist1_c5.err
timeout 600 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/${TAG}_bench_reference.json 2> gpurun_out/${TAG}_bench_reference.err
bash tools/profile_round.sh ${TAG} c4_u64_2p28
rm -f gpurun_out/prof_${TAG}_k_classify.ncu-rep
