set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 600 python bench.py > gpurun_out/r02t_bench.json 2> gpurun_out/r02t_bench.err
tail -c 2500 gpurun_out/r02t_bench.json
timeout 300 python -c "
import torch,time
x=torch.randint(-2**62,2**62,(1<<28,),dtype=torch.int64,device='cuda')
for i in range(3): y=torch.sort(x)[0]
torch.cuda.synchronize()
e0=torch.cuda.Event(enable_timing=True);e1=torch.cuda.Event(enable_timing=True)
e0.record()
for i in range(5): y=torch.sort(x)[0]
e1.record();torch.cuda.synchronize()
print('torch.sort int64 2^28 ms',e0.elapsed_time(e1)/5)
x=x.to(torch.int32)
for i in range(3): y=torch.sort(x)[0]
e0.record()
for i in range(5): y=torch.sort(x)[0]
e1.record();torch.cuda.synchronize()
print('torch.sort int32 2^28 ms',e0.elapsed_time(e1)/5)
" > gpurun_out/r02t_torchsort.log 2>&1
bash tools/ncu_one.sh r02t k_small_block 4
bash tools/ncu_one.sh r02t k_scatter_bulk 0
bash tools/ncu_one.sh r02t k_classify 1
ls -la gpurun_out
