bash tools/ncu_one.sh r02ae k_scatter_ws 0
bash tools/ncu_one.sh r02ae k_classify 1
