"""Summarise an ncu source page (SASS) : instruction mix and stall samples by opcode / top instructions."""
import csv, sys, collections, subprocess
rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"], capture_output=True, text=True).stdout
r = list(csv.reader(out.splitlines()))
h = r[1]; rows = r[2:]
ie = h.index("Instructions Executed"); ws = h.index("Warp Stall Sampling (All Samples)"); src = h.index("Source")
wf = h.index("L1 Wavefronts Shared"); wfi = h.index("L1 Wavefronts Shared Ideal")
tot = sum(float(x[ie] or 0) for x in rows); tws = sum(float(x[ws] or 0) for x in rows)
by = collections.defaultdict(lambda: [0.0, 0.0, 0.0, 0.0])
for x in rows:
    op = x[src].strip().split()[0] if x[src].strip() else "?"
    if op.startswith("@"):
        op = x[src].strip().split()[1]
    op = op.split(".")[0]
    by[op][0] += float(x[ie] or 0); by[op][1] += float(x[ws] or 0)
    by[op][2] += float(x[wf] or 0); by[op][3] += float(x[wfi] or 0)
print(f"total warp-instructions executed: {tot:.4g}; stall samples {tws:.4g}")
for op, (i, s, w, wi) in sorted(by.items(), key=lambda kv: -kv[1][1])[:22]:
    print(f"{op:10s} inst {i/tot*100:5.1f}%  stall {s/tws*100:5.1f}%  smem wavefronts {w:.3g} (ideal {wi:.3g})")
print("--- top instructions by stall samples")
rows.sort(key=lambda x: -float(x[ws] or 0))
for x in rows[:int(sys.argv[2]) if len(sys.argv) > 2 else 20]:
    print(f"{x[0][-5:]} stall {float(x[ws])/tws*100:5.1f}% inst {float(x[ie])/tot*100:4.1f}%  {x[src].strip()[:90]}")
