"""Do two independent sorts on two streams overlap?  (probe for kernel-level concurrency)"""
import os, sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch, inputs
import paper_conf_ipps_leischneros10_b200 as gss
n = 1 << 27
xs = [torch.from_numpy(inputs.keys("uniform", n, 64, seed=s)).cuda() for s in (1, 2)]
outs = [torch.empty_like(x) for x in xs]
sorters = [gss.Sorter("u64", n, k=256, tile=32768) for _ in range(2)]
streams = [torch.cuda.Stream() for _ in range(2)]
def seq():
    for i in range(2):
        sorters[i](xs[i], outs[i])
def par():
    for i in range(2):
        with torch.cuda.stream(streams[i]):
            sorters[i](xs[i], outs[i], stream=streams[i])
for name, f in (("sequential", seq), ("two streams", par)):
    for _ in range(2):
        f()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(5):
        f()
    for s in streams:
        torch.cuda.current_stream().wait_stream(s)
    e1.record()
    torch.cuda.synchronize()
    print(name, e0.elapsed_time(e1) / 5, "ms for two 2^27 sorts")
