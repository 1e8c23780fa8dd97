"""Per-source-line summary of an ncu report's source page (cuda,sass view): warp-level
instructions executed and warp-stall samples by line, for one launch.

    python tools/ncu_lines.py REPORT.ncu-rep [--launch I] [--top 40]
"""
import argparse
import csv
import io
import subprocess

ap = argparse.ArgumentParser()
ap.add_argument("report")
ap.add_argument("--launch", type=int, default=0)
ap.add_argument("--top", type=int, default=40)
ap.add_argument("--rows", type=float, default=0, help="divide instructions by rows (per-row cost)")
a = ap.parse_args()
out = subprocess.run(["ncu", "-i", a.report, "--page", "source", "--csv", "--print-source", "cuda,sass",
                      "--launch-skip", str(a.launch), "--launch-count", "1"],
                     capture_output=True, text=True).stdout
fname, hdr, lines = None, None, []
for row in csv.reader(io.StringIO(out)):
    if not row:
        continue
    if row[0] == "File Path":
        fname = row[1].split("/")[-1]
    elif row[0] == "Line No":
        hdr = row
    elif hdr and row[0].isdigit():
        d = dict(zip(hdr[2:], row[2:]))  # (the second "Source" column shadows; skip Address)
        try:
            samp = int(d.get("Warp Stall Sampling (All Samples)", "0") or 0)
            inst = int(d.get("Instructions Executed", "0") or 0)
        except ValueError:
            continue
        stalls = {k[6:]: int(v) for k, v in d.items() if k.startswith("stall_") and v.isdigit() and int(v) > 0}
        lines.append((samp, inst, f"{fname}:{row[0]}", row[1][:70], stalls))
tot_s = sum(x[0] for x in lines) or 1
tot_i = sum(x[1] for x in lines) or 1
print(f"total samples {tot_s}, warp instructions {tot_i}" +
      (f" ({tot_i / a.rows:.2f} warp-instr/row)" if a.rows else ""))
for samp, inst, where, src, stalls in sorted(lines, reverse=True)[: a.top]:
    top = sorted(stalls.items(), key=lambda kv: -kv[1])[:3]
    print(f"{100 * samp / tot_s:5.1f}% samp {100 * inst / tot_i:5.1f}% inst  {where:22s} {src:70s} "
          + " ".join(f"{k}={v}" for k, v in top))
