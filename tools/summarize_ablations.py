"""Summarise the ablation captures of tools/ncu_ablations.sh (gpurun_out/abl_<tag>_*.ncu-rep) into
gpurun_out/abl_<tag>_summary.{json,md}: duration, DRAM bytes, instructions, shared-memory wavefronts and bank
conflicts, issue activity, divergence, per variant.  usage: python tools/summarize_ablations.py <tag>"""
import csv, glob, json, os, subprocess, sys

tag = sys.argv[1]
G = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "gpurun_out")
M = {
    "duration_ms": ("gpu__time_duration.sum", 1e-6),
    "dram_read_GB": ("dram__bytes_read.sum", 1e-9),
    "dram_write_GB": ("dram__bytes_write.sum", 1e-9),
    "inst_executed": ("smsp__inst_executed.sum", 1),
    "issue_active_pct": ("smsp__issue_active.avg.pct_of_peak_sustained_active", 1),
    "warps_active_pct": ("sm__warps_active.avg.pct_of_peak_sustained_active", 1),
    "smem_wavefronts": ("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", 1),
    "smem_ld_bank_conflicts": ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", 1),
    "smem_st_bank_conflicts": ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum", 1),
    "atom_bank_conflicts": ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_atom.sum", 1),
    "branch_targets": ("smsp__sass_branch_targets.sum", 1),
    "branch_targets_divergent": ("smsp__sass_branch_targets_threads_divergent.sum", 1),
    "threads_per_inst": ("smsp__thread_inst_executed_per_inst_executed.ratio", 1),
    "registers": ("launch__registers_per_thread", 1),
}
UNITS = {"ms": 1e-3, "us": 1e-6, "ns": 1e-9, "s": 1.0, "byte": 1.0, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
out = {}
for rep in sorted(glob.glob(os.path.join(G, f"abl_{tag}_*.ncu-rep"))):
    name = os.path.basename(rep)[len(f"abl_{tag}_"):-len(".ncu-rep")]
    txt = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(txt.splitlines()))
    if len(rows) < 3:
        continue
    h, u, v = rows[0], rows[1], rows[2]
    d = {"kernel": v[h.index("Kernel Name")] if "Kernel Name" in h else ""}
    for key, (metric, scale) in M.items():
        if metric in h:
            i = h.index(metric)
            try:
                x = float(v[i].replace(",", ""))
            except ValueError:
                continue
            unit = u[i]
            if key == "duration_ms":
                x = x * UNITS.get(unit, 1e-9) / 1e-3
            elif key.endswith("_GB"):
                x = x * UNITS.get(unit, 1.0) / 1e9
            d[key] = round(x, 4) if isinstance(x, float) else x
    if d.get("smem_wavefronts"):
        d["bank_conflict_frac"] = round((d.get("smem_ld_bank_conflicts", 0) + d.get("smem_st_bank_conflicts", 0)) /
                                        d["smem_wavefronts"], 4)
    out[name] = d
json.dump(out, open(os.path.join(G, f"abl_{tag}_summary.json"), "w"), indent=1)
with open(os.path.join(G, f"abl_{tag}_summary.md"), "w") as f:
    cols = ["duration_ms", "dram_read_GB", "dram_write_GB", "inst_executed", "issue_active_pct", "warps_active_pct",
            "smem_wavefronts", "bank_conflict_frac", "branch_targets_divergent", "registers"]
    f.write(f"# ablation ncu counters ({tag}; 2^28 uniform u64, one launch each, cold, serialised)\n\n")
    f.write("| variant | " + " | ".join(cols) + " |\n|" + "---|" * (len(cols) + 1) + "\n")
    for name, d in out.items():
        f.write(f"| {name} | " + " | ".join(str(d.get(c, "")) for c in cols) + " |\n")
print(json.dumps(out, indent=1))
