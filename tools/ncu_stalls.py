"""Key counters + stall reasons of an ncu report (first kernel)."""
import csv, subprocess, sys
rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
r = list(csv.reader(out.splitlines()))
h = r[0]; v = r[2]
d = dict(zip(h, v))
items = [(k, d[k]) for k in h if k.startswith('smsp__average_warps_issue_stalled') and k.endswith('_per_issue_active.ratio')]
items.sort(key=lambda kv: -float(kv[1].replace(',', '') or 0))
print("stalls/issue:", ", ".join(f"{k.replace('smsp__average_warps_issue_stalled_','').replace('_per_issue_active.ratio','')}={float(x):.2f}" for k, x in items[:8]))
keys = ['gpu__time_duration.sum', 'smsp__inst_executed.sum', 'smsp__issue_active.avg.pct_of_peak_sustained_active',
        'sm__warps_active.avg.pct_of_peak_sustained_active', 'launch__registers_per_thread', 'launch__grid_size',
        'launch__block_size', 'launch__occupancy_limit_registers', 'launch__occupancy_limit_shared_mem',
        'dram__throughput.avg.pct_of_peak_sustained_elapsed', 'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum',
        'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum', 'l1tex__data_pipe_lsu_wavefronts_mem_shared.sum',
        'smsp__sass_branch_targets_threads_divergent.sum', 'smsp__sass_branch_targets.sum',
        'smsp__thread_inst_executed_per_inst_executed.ratio', 'dram__bytes_read.sum', 'dram__bytes_write.sum']
for k in keys:
    if k in d:
        print(f"  {k} = {d[k]}")
