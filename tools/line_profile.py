"""Map an ncu SASS source page onto CUDA source lines using nvdisasm line info.
usage: python tools/line_profile.py <report.ncu-rep> <libgss.so or cubin> [top]
The .so must be the one that was profiled (gpu_quick.sh copies it as gpurun_out/libgss_<tag>.so)."""
import collections, csv, os, re, subprocess, sys, tempfile

rep, lib = sys.argv[1], sys.argv[2]
top = int(sys.argv[3]) if len(sys.argv) > 3 else 30
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
kname = rows[0][1]
h = rows[1]; data = rows[2:]
ie, ws, src = h.index("Instructions Executed"), h.index("Warp Stall Sampling (All Samples)"), h.index("Source")
base = int(data[0][0], 16)
# mangled name: ask ncu for it
raw = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv", "--metrics", "launch__grid_size"],
                     capture_output=True, text=True).stdout
# find the function in the cubin by matching the demangled kernel name
tmp = tempfile.mkdtemp()
if lib.endswith(".so"):
    subprocess.run(["cuobjdump", "-xelf", "all", os.path.abspath(lib)], cwd=tmp, capture_output=True)
    cubs = [os.path.join(tmp, f) for f in sorted(os.listdir(tmp)) if f.endswith(".cubin")]
else:
    cubs = [lib]
sass = []
for cub in cubs:   # libgss.so holds one cubin per translation unit
    sass += subprocess.run(["nvdisasm", "-g", "-c", cub], capture_output=True, text=True).stdout.splitlines()
# split functions
funcs = {}
cur = None
for line in sass:
    m = re.match(r"^\s*\.text\.(\S+):", line)
    if m:
        cur = m.group(1); funcs[cur] = []; continue
    if cur is not None:
        funcs[cur].append(line)
# pick function whose demangled name matches the kernel name
def dem(n):
    return subprocess.run(["c++filt", n], capture_output=True, text=True).stdout.strip()
target = None
def norm(s):
    s = s.split("(gss::Ctx")[0]
    s = s.replace("(bool)0", "false").replace("(bool)1", "true")
    return re.sub(r"\(int\)|\s+", "", s)
kn = norm(kname)
for f in funcs:
    if norm(dem(f)) == kn:
        target = f; break
if target is None:
    print("function not found for", kname); sys.exit(1)
off2line = {}
cur_line = ("?", 0)
for line in funcs[target]:
    m = re.search(r'//## File "([^"]+)", line (\d+)', line)
    if m:
        cur_line = (os.path.basename(m.group(1)), int(m.group(2)))
        continue
    m = re.search(r"/\*([0-9a-f]{4,})\*/", line)
    if m:
        off2line[int(m.group(1), 16)] = cur_line
agg = collections.defaultdict(lambda: [0.0, 0.0])
ti = ts = 0.0
for r in data:
    off = int(r[0], 16) - base
    ln = off2line.get(off, ("?", 0))
    i, s = float(r[ie] or 0), float(r[ws] or 0)
    agg[ln][0] += i; agg[ln][1] += s; ti += i; ts += s
print(kname[:120])
print(f"total warp-instructions {ti:.4g}, stall samples {ts:.4g}")
for (f, l), (i, s) in sorted(agg.items(), key=lambda kv: -kv[1][int(os.environ.get("LP_SORT_STALL", "1"))])[:top]:
    print(f"{f}:{l:<5d} inst {i/ti*100:5.1f}%  stall {s/ts*100:5.1f}%")
