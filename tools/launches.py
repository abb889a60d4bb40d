"""Print an ncu launch list (gpu__time_duration + dram bytes) of the last sort in a log."""
import csv, collections, sys
rows = list(csv.reader(open(sys.argv[1])))
hi = [i for i, r in enumerate(rows) if r and r[0] == 'ID'][0]
h = rows[hi]; data = rows[hi + 1:]
ki, mi, vi, idi = h.index('Kernel Name'), h.index('Metric Name'), h.index('Metric Value'), h.index('ID')
recs = collections.OrderedDict()
for r in data:
    recs.setdefault(r[idi], {'name': r[ki]})[r[mi]] = float(r[vi].replace(',', ''))
items = list(recs.values())
# the last sort: from the last k_init
last = max(i for i, v in enumerate(items) if 'k_init' in v['name'])
tot = 0
for v in items[last:]:
    t = v.get('gpu__time_duration.sum', 0); tot += t
    nm = v['name'].split('(')[0].replace('void gss::', '')[:70]
    print(f"{t/1e3:9.1f} us  rd {v.get('dram__bytes_read.sum',0)/1e9:7.3f} GB  wr {v.get('dram__bytes_write.sum',0)/1e9:7.3f} GB  {nm}")
print(f"total {tot/1e6:.3f} ms")
