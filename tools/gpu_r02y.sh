bash tools/ncu_one.sh r02y k_scatter_ws 0
