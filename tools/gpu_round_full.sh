#!/bin/bash
# Everything a round needs from the GPU: full gpu tests, smoke, bench lines of every workload, launch list,
# full ncu captures.  usage: tools/gpu_round_full.sh <tag>
TAG=${1:-r01}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/smi_${TAG}.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_${TAG}.log 2>&1
echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests_${TAG}.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_${TAG}.log 2>&1; echo "smoke rc=$?"
timeout 600 python bench.py > gpurun_out/bench_${TAG}_c4_u64_2p28.json 2> gpurun_out/bench_${TAG}_c4_u64_2p28.err; echo "bench rc=$?"
for WL in c2_u32_2p27 c3_u64_2p27 c3_kv64_2p27 c1_u32_2p16 c4_u64_2p29 c4_u64_2p30; do
  timeout 600 python bench.py --workload $WL --no-cpu-baseline > gpurun_out/bench_${TAG}_${WL}.json 2> gpurun_out/bench_${TAG}_${WL}.err
  echo "bench $WL rc=$?"
done
timeout 300 python bench.py --force-dist --no-cpu-baseline > gpurun_out/bench_${TAG}_dist_force1.json 2> gpurun_out/bench_${TAG}_dist.err
echo "bench dist rc=$?"
tools/profile_round.sh $TAG c4_u64_2p28
rm -f gpurun_out/prof_${TAG}_k_classify.ncu-rep gpurun_out/prof_${TAG}_k_scatter.ncu-rep.bak
