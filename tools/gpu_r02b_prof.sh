set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,driver_version --format=csv > gpurun_out/r02b_smi.txt
bash tools/profile_round.sh r02b c4_u64_2p28
ls -la gpurun_out | tail -20
