"""Top SASS instructions of an ncu report by stall samples, with the stall reasons.
usage: python tools/sass_stalls.py <report.ncu-rep> [top]"""
import csv, subprocess, sys
rep = sys.argv[1]; top = int(sys.argv[2]) if len(sys.argv) > 2 else 25
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]; data = rows[2:]
ia, isrc, iw = h.index("Address"), h.index("Source"), h.index("Warp Stall Sampling (All Samples)")
ie = h.index("Instructions Executed")
st = [i for i, c in enumerate(h) if c.startswith("stall_") and "Not Issued" not in c]
tot = sum(float(r[iw] or 0) for r in data)
base = int(data[0][ia], 16)
for r in sorted(data, key=lambda r: -float(r[iw] or 0))[:top]:
    reasons = sorted(((h[i][6:], float(r[i] or 0)) for i in st), key=lambda x: -x[1])[:3]
    rs = " ".join(f"{n}={v/ max(float(r[iw]),1)*100:.0f}%" for n, v in reasons if v)
    print(f"{int(r[ia],16)-base:6x} {float(r[iw])/tot*100:5.1f}% inst={int(float(r[ie])):>10}  {r[isrc].strip()[:60]:60s} {rs}")
