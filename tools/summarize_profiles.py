"""Summarise an ncu K1 capture + a launch list into profiles/ (markdown + k1_traffic.json).

    python tools/summarize_profiles.py <tag> <k1.ncu-rep> <launches.csv>
"""
import collections
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
QS = ["q1.1", "q1.2", "q1.3", "q2.1", "q2.2", "q2.3", "q3.1", "q3.2", "q3.3", "q3.4", "q4.1", "q4.2", "q4.3"]
N = 60_000_000
BROW = {"1": 16, "2": 16, "3": 16, "4": 24}


def main(tag, rep, launches):
    raw = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    hdr, data = rows[0], rows[2:]
    c = hdr.index
    out = [f"# {tag} — ncu --set full of K1 (k1_probe_agg), SSB SF10, 1 B200", "",
           "Captured with `ncu --set full --clock-control none --import-source on -k regex:k1_probe_agg "
           "-s 13 -c 13 python tools/prof_query.py --sf 10 --queries all --reps 2` (the second, "
           "planned execution of each query). ncu times are cold-cache and serialised: compare shares.", "",
           "| query | kernel | ncu us | algorithmic GB | DRAM r+w GB | traffic/alg | DRAM GB/s (% of 8 TB/s) | L2 hit % | issue active % | warps active % | regs |",
           "|---|---|---|---|---|---|---|---|---|---|---|"]
    def scaled(d, name):  # ncu raw values carry their unit in the second header row
        unit = rows[1][c(name)]
        mult = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9}
        return float(d[c(name)] or 0) * mult.get(unit, 1)

    tt = ta = tr = 0.0
    for q, d in zip(QS, data):
        t = float(d[c("gpu__time_duration.sum")])
        rd = scaled(d, "dram__bytes_read.sum")
        wr = scaled(d, "dram__bytes_write.sum")
        alg = N * BROW[q[1]]
        tt, ta, tr = tt + t, ta + alg, tr + rd + wr
        out.append(f"| {q} | {d[c('Kernel Name')].split('(')[0].split('::')[-1]} | {t:.1f} | {alg/1e9:.3f} | "
                   f"{(rd+wr)/1e9:.3f} | {(rd+wr)/alg:.3f} | {(rd+wr)/(t*1e3):.0f} ({(rd+wr)/(t*1e3)/80:.0f}%) | "
                   f"{float(d[c('lts__t_sector_hit_rate.pct')]):.1f} | "
                   f"{float(d[c('smsp__issue_active.avg.pct_of_peak_sustained_active')]):.1f} | "
                   f"{float(d[c('sm__warps_active.avg.pct_of_peak_sustained_active')]):.1f} | "
                   f"{d[c('launch__registers_per_thread')]} |")
    out += ["", f"Sum over the 13 launches: {tt:.0f} us; algorithmic {ta/1e9:.2f} GB; DRAM {tr/1e9:.2f} GB "
                f"(traffic/algorithmic {tr/ta:.3f}; below 1 where late materialisation gathers measure columns for passing rows only)."]
    with open(os.path.join(ROOT, "profiles", f"{tag}_k1_ncu_summary.md"), "w") as f:
        f.write("\n".join(out) + "\n")
    with open(os.path.join(ROOT, "profiles", "k1_traffic.json"), "w") as f:
        json.dump({"dram_bytes_per_launch": tr / 13, "algorithmic_bytes_per_launch": ta / 13,
                   "launches": 13, "source": f"profiles/{tag}_k1_ncu_summary.md (ncu --set full, "
                   "dram__bytes_read.sum + dram__bytes_write.sum, mean over the 13 SSB K1 launches at SF10)"}, f, indent=1)
    rows = list(csv.reader(open(launches)))
    h = [i for i, r in enumerate(rows) if "Kernel Name" in r][0]
    hd = rows[h]
    agg, cnt = collections.Counter(), collections.Counter()
    for r in rows[h + 1:]:
        name = r[hd.index("Kernel Name")].split("(")[0].split("::")[-1].split("<")[0]
        agg[name] += float(r[hd.index("Metric Value")].replace(",", ""))
        cnt[name] += 1
    tot = sum(agg.values())
    L = [f"# {tag} — launch list of `bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline`",
         "", "ncu `gpu__time_duration.sum --clock-control none` over every launch of the run (plan "
         "creation, warm-up, timed steps, per-query pass); serialised and cold: SHARES only.", "",
         "| kernel | launches | total us | share |", "|---|---|---|---|"]
    for k, v in agg.most_common():
        L.append(f"| {k} | {cnt[k]} | {v/1e3:.1f} | {100*v/tot:.1f}% |")
    with open(os.path.join(ROOT, "profiles", f"{tag}_launch_shares.md"), "w") as f:
        f.write("\n".join(L) + "\n")
    print("\n".join(out[-1:] + L[-len(agg):]))


if __name__ == "__main__":
    main(*sys.argv[1:4])
