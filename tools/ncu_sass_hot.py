"""Per-SASS-line executed warp instructions and stall samples from an ncu report:
python tools/ncu_sass_hot.py rep.ncu-rep [top]   (prints the hottest lines and a
per-opcode histogram of executed instructions)"""
import collections
import csv
import io
import subprocess
import sys

rep = sys.argv[1]
top = int(sys.argv[2]) if len(sys.argv) > 2 else 40
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
lines = out.splitlines()
rows = list(csv.reader(io.StringIO("\n".join(lines[1:]))))
hdr = rows[0]
ix = {h: i for i, h in enumerate(hdr)}
data = []
for r in rows[1:]:
    try:
        data.append((int(r[ix["Instructions Executed"]]), int(r[ix["Warp Stall Sampling (All Samples)"]]),
                     r[ix["Address"]], r[ix["Source"]].strip()))
    except (ValueError, IndexError):
        pass
tot = sum(d[0] for d in data)
stall = sum(d[1] for d in data)
print(f"total warp instructions {tot}, stall samples {stall}")
op = collections.Counter()
for n, s, a, src in data:
    o = src.split()[0] if not src.startswith("@") else src.split()[1]
    op[o.split(".")[0]] += n
for o, n in op.most_common(25):
    print(f"  {o:10s} {n:12d} {n / tot:6.1%}")
print("hottest lines by stall samples:")
for n, s, a, src in sorted(data, key=lambda d: -d[1])[:top]:
    print(f"  {s:6d} {n:10d}  {src[:90]}")
