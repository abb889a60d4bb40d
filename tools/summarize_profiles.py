"""Summarise a round's ncu captures into profiles/<tag>_ncu_summary.{json,md}.
usage: python tools/summarize_profiles.py <tag> <workload> <libgss.so used>"""
import csv, json, os, subprocess, sys
tag, wl, lib = sys.argv[1], sys.argv[2], sys.argv[3]
OUTDIR = sys.argv[4] if len(sys.argv) > 4 else None
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
G = os.path.join(ROOT, "gpurun_out")
METRICS = {
    "duration_ms": ("gpu__time_duration.sum", 1e-6),
    "dram_read_GB": ("dram__bytes_read.sum", 1e-9),
    "dram_write_GB": ("dram__bytes_write.sum", 1e-9),
    "dram_throughput_pct": ("dram__throughput.avg.pct_of_peak_sustained_elapsed", 1),
    "issue_active_pct": ("smsp__issue_active.avg.pct_of_peak_sustained_active", 1),
    "warps_active_pct": ("sm__warps_active.avg.pct_of_peak_sustained_active", 1),
    "inst_executed": ("smsp__inst_executed.sum", 1),
    "smem_wavefronts": ("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", 1),
    "smem_ld_bank_conflicts": ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", 1),
    "smem_st_bank_conflicts": ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum", 1),
    "branch_targets": ("smsp__sass_branch_targets.sum", 1),
    "branch_targets_divergent": ("smsp__sass_branch_targets_threads_divergent.sum", 1),
    "threads_per_inst": ("smsp__thread_inst_executed_per_inst_executed.ratio", 1),
    "pipe_alu_pct": ("sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active", 1),
    "pipe_fma_pct": ("sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active", 1),
    "pipe_lsu_pct": ("sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active", 1),
    "smem_pipe_pct": ("l1tex__data_pipe_lsu_wavefronts_mem_shared.avg.pct_of_peak_sustained_elapsed", 1),
    "registers": ("launch__registers_per_thread", 1),
    "block": ("launch__block_size", 1),
    "grid": ("launch__grid_size", 1),
}
out = {"tag": tag, "workload": wl, "kernels": {}}
for k in ("k_classify", "k_scatter", "k_small"):
    rep = os.path.join(G, f"prof_{tag}_{k}.ncu-rep")
    if not os.path.exists(rep):
        continue
    raw = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    r = list(csv.reader(raw.splitlines()))
    d = dict(zip(r[0], r[2]))
    unit = dict(zip(r[0], r[1]))
    e = {"kernel": d.get("Kernel Name", "")[:160]}
    for name, (m, scale) in METRICS.items():
        if m in d and d[m] not in ("", "n/a"):
            v = float(d[m].replace(",", ""))
            u = unit.get(m, "")
            if m.startswith("dram__bytes"):
                v = v * {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9}.get(u, 1)
            if m == "gpu__time_duration.sum":
                v = v * {"nsecond": 1, "ns": 1, "usecond": 1e3, "us": 1e3, "msecond": 1e6, "ms": 1e6}.get(u, 1)
            e[name] = v * scale
    if "duration_ms" in e and "dram_read_GB" in e:
        e["dram_GBps"] = (e["dram_read_GB"] + e["dram_write_GB"]) / (e["duration_ms"] * 1e-3)
    if e.get("branch_targets"):
        e["divergent_branch_pct"] = 100.0 * e.get("branch_targets_divergent", 0) / e["branch_targets"]
    stalls = [(kk, float(d[kk])) for kk in r[0] if kk.startswith("smsp__average_warps_issue_stalled") and
              kk.endswith("_per_issue_active.ratio") and d[kk]]
    stalls.sort(key=lambda x: -x[1])
    e["top_stalls_per_issue"] = {kk.replace("smsp__average_warps_issue_stalled_", "").replace(
        "_per_issue_active.ratio", ""): round(v, 2) for kk, v in stalls[:6]}
    lp = subprocess.run([sys.executable, os.path.join(ROOT, "tools", "line_profile.py"), rep, lib, "12"],
                        capture_output=True, text=True).stdout
    e["hot_source_lines"] = lp.strip().splitlines()[2:]
    out["kernels"][k] = e
lcsv = os.path.join(G, f"launches_{tag}_{wl}.csv")
if os.path.exists(lcsv):
    out["launch_list"] = subprocess.run([sys.executable, os.path.join(ROOT, "tools", "launches.py"), lcsv],
                                        capture_output=True, text=True).stdout.strip().splitlines()
odir = OUTDIR or os.path.join(ROOT, "profiles")
json.dump(out, open(os.path.join(odir, f"{tag}_ncu_summary.json"), "w"), indent=1)
with open(os.path.join(odir, f"{tag}_ncu_summary.md"), "w") as f:
    f.write(f"# ncu summary {tag} — workload {wl}\n\n")
    f.write("Captured with `ncu --set full --clock-control none` (one launch each; cold, serialised: compare shares, "
            "not absolute times).\n\n")
    for k, e in out["kernels"].items():
        f.write(f"## {k}\n\n`{e['kernel']}`\n\n")
        for name in ("duration_ms", "dram_read_GB", "dram_write_GB", "dram_GBps", "dram_throughput_pct",
                     "issue_active_pct", "warps_active_pct", "inst_executed", "smem_wavefronts",
                     "smem_ld_bank_conflicts", "smem_st_bank_conflicts", "divergent_branch_pct", "pipe_alu_pct", "pipe_fma_pct", "pipe_lsu_pct", "smem_pipe_pct",
                     "threads_per_inst", "registers", "block", "grid"):
            if name in e:
                v = e[name]
                f.write(f"- {name}: {v:.4g}\n" if isinstance(v, float) else f"- {name}: {v}\n")
        f.write(f"- top stalls (warps per issue): {e['top_stalls_per_issue']}\n\n")
        f.write("Hot source lines (share of instructions / stall samples):\n\n```\n" +
                "\n".join(e["hot_source_lines"]) + "\n```\n\n")
    if "launch_list" in out:
        f.write("## Launch list of one sort (ncu gpu__time_duration, dram bytes)\n\n```\n" +
                "\n".join(out["launch_list"]) + "\n```\n")
print("wrote", os.path.join(odir, f"{tag}_ncu_summary.md"))
