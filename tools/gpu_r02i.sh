set -x
timeout 600 python bench.py > gpurun_out/r02i_bench.json 2> gpurun_out/r02i_bench.err
bash tools/profile_round.sh r02i c4_u64_2p28
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/r02i_smi.txt
