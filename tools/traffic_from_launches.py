"""Per-kind DRAM bytes of one sort from an ncu launch list (the last sort in the csv) ->
profiles/ncu_traffic_<workload>.json, which bench.py reports as roofline.traffic.
usage: python tools/traffic_from_launches.py <launches.csv> <workload> <source note>"""
import collections, csv, json, os, sys
rows = list(csv.reader(open(sys.argv[1])))
hi = [i for i, r in enumerate(rows) if r and r[0] == 'ID'][0]
h = rows[hi]; data = rows[hi + 1:]
ki, mi, vi, idi = h.index('Kernel Name'), h.index('Metric Name'), h.index('Metric Value'), h.index('ID')
recs = collections.OrderedDict()
for r in data:
    recs.setdefault(r[idi], {'name': r[ki]})[r[mi]] = float(r[vi].replace(',', ''))
items = list(recs.values())
last = max(i for i, v in enumerate(items) if 'k_init' in v['name'])
KIND = [("k_init", "init"), ("k_sample", "sample"), ("k_set_splitters", "sample"), ("k_classify", "classify"),
        ("k_scan", "scan"), ("k_scatter", "scatter"), ("k_plan", "plan"), ("k_small", "small_sort"),
        ("k_copy", "copy"), ("k_overflow", "overflow")]
out = collections.OrderedDict((k, 0.0) for _, k in KIND)
for v in items[last:]:
    nm = v['name'].split('(')[0]
    for pre, kind in KIND:
        if pre in nm:
            out[kind] += v.get('dram__bytes_read.sum', 0) + v.get('dram__bytes_write.sum', 0)
            break
out["_note"] = ("dram__bytes_read.sum + dram__bytes_write.sum summed over all launches of each kernel kind in "
                f"one sort ({sys.argv[3]}); bytes per step")
root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
json.dump(out, open(os.path.join(root, "profiles", f"ncu_traffic_{sys.argv[2]}.json"), "w"), indent=1)
print(json.dumps(out))
