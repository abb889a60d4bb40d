timeout 900 python -m pytest tests/test_gpu_sort.py -m gpu -x -q -p no:cacheprovider -k "sort_distributions" > gpurun_out/r02ai_pytest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r02ai_pytest.log
for wl in c3_kv64_2p27 c5_kv64_2p29; do
  timeout 600 python tools/sweep.py --workload $wl k=0 k=0,flags=67108864 k=0 k=0,flags=67108864 >> gpurun_out/r02ai_ab.log 2>&1
done
for d in sorted dd and4; do GSS_DIST=$d timeout 300 python tools/sweep.py --workload c3_kv64_2p27 k=0 k=0,flags=67108864 >> gpurun_out/r02ai_ab.log 2>&1; done
python - <<'PY'
import sys; sys.path.insert(0,'.')
import numpy as np, torch, inputs, oracle, paper_conf_ipps_leischneros10_b200 as gss
from tests.test_gpu_sort import check_pairs
for n in ((1<<20)+4321, (1<<22)+77):
    for dist in ("uniform","dd","and3","sorted"):
        x = inputs.keys(dist, n, 64, seed=1); v = inputs.values(n, 64)
        ko, vo = gss.sort(torch.from_numpy(x).cuda(), torch.from_numpy(v).cuda(), M=4096, flags=67108864)
        ok,_ = oracle.sort(x, None, oracle.Params(k=256,a=30,M=4096,k_policy=1,fill_div=4,seed=5489))
        assert np.array_equal(ko.cpu().numpy(), ok), (n, dist)
        check_pairs(x, vo.cpu().numpy(), ok)
print("ws-one pairs parity ok")
PY
