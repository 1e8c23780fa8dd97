"""ncu summary of the K3 hash-pack kernels -> profiles/<tag>_k3_ncu_summary.md

    python tools/summarize_k3.py <tag> <k3.ncu-rep>
"""
import csv
import io
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
tag, rep = sys.argv[1], sys.argv[2]
raw = (open(rep).read() if rep.endswith(".csv") else  # a saved `--page raw --csv` export
       subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout)
rows = list(csv.reader(io.StringIO(raw)))
hdr, units, data = rows[0], rows[1], rows[2:]
c = hdr.index
MULT = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1e-3, "usecond": 1,
        "msecond": 1e3, "ns": 1e-3, "us": 1, "ms": 1e3}


def val(d, name):
    return float(d[c(name)] or 0) * MULT.get(units[c(name)], 1)


L = [f"# {tag} — ncu --set full of K3 (hash-pack, §8(f) NEXT-1): 600 M rows × 6 columns into 8 parts (SF100)", "",
     "`ncu --set full --clock-control none -k regex:k3_ -c 3 python tools/hashpack_bench.py --sf 100 "
     "--parts 8 --reps 1` (cold caches, serialised). r02: the scatter stages its tiles with "
     "cp.async.bulk (k3_scatter_tma).", "",
     "| kernel | us | DRAM read GB | DRAM write GB | DRAM GB/s (% of 8 TB/s) | issue active % | L2 hit % |",
     "|---|---|---|---|---|---|---|"]
for d in data:
    t = val(d, "gpu__time_duration.sum")
    rd, wr = val(d, "dram__bytes_read.sum"), val(d, "dram__bytes_write.sum")
    name = d[c("Kernel Name")].split("(")[0].split("::")[-1]
    L.append(f"| {name} | {t:.0f} | {rd/1e9:.2f} | {wr/1e9:.2f} | {(rd+wr)/(t*1e3):.0f} ({(rd+wr)/(t*1e3)/80:.0f}%) | "
             f"{float(d[c('smsp__issue_active.avg.pct_of_peak_sustained_active')]):.1f} | "
             f"{float(d[c('lts__t_sector_hit_rate.pct')]):.1f} |")
L += ["", "Algorithmic bytes: count reads the key column (2.4 GB); scatter reads 6 columns (14.4 GB) "
      "and writes them (14.4 GB)."]
open(os.path.join(ROOT, "profiles", f"{tag}_k3_ncu_summary.md"), "w").write("\n".join(L) + "\n")
print("\n".join(L))
