set -x
bash tools/ncu_ablations.sh r02n
timeout 600 python tools/sweep.py --workload c4_u64_2p28 flags=16 a=15,flags=16 a=20,flags=16 > gpurun_out/r02n_sweep_a.log 2>&1
du -sh gpurun_out
