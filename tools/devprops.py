"""Record the B200 device properties the design depends on."""
import json, subprocess, torch
p = torch.cuda.get_device_properties(0)
out = {k: getattr(p, k) for k in dir(p) if not k.startswith('_') and isinstance(getattr(p, k), (int, float, str, bool))}
out["torch"] = torch.__version__
try:
    out["nvidia_smi"] = subprocess.run(["nvidia-smi", "--query-gpu=name,memory.total,clocks.max.sm,clocks.max.mem,power.limit", "--format=csv"], capture_output=True, text=True).stdout
except Exception as e:
    out["nvidia_smi"] = str(e)
import os
out["host_cpus"] = os.cpu_count()
try:
    out["cpu_model"] = [l for l in open('/proc/cpuinfo') if l.startswith('model name')][0].split(':')[1].strip()
except Exception:
    pass
print(json.dumps(out, indent=1, default=str))
json.dump(out, open("gpurun_out/devprops.json", "w"), indent=1, default=str)
