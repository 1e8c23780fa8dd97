"""Summarise an ncu K1 capture + a launch list into profiles/ (markdown + k1_traffic.json).

    python tools/summarize_profiles.py <tag> <k1.ncu-rep> <launches.csv> [SF] [probe_l2.csv]

probe_l2.csv (optional): an ncu --csv metrics list of the 13 K1 launches built with probe loads
tagged evict_last (HX_PROBE_HINT=1) and gathers evict_first: the evict_last L2 sectors are then
exactly the probe-structure lookups, so their hit rate is the probe tables' L2 hit rate.
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
N = 60_000_000  # rows (SF10); main() takes the SF
BROW = {"1": 16, "2": 16, "3": 16, "4": 24}


def main(tag, rep, launches, sf="10", probe_csv=None):
    global N
    launches = None if launches == "-" else launches
    N = int(6_000_000 * float(sf))
    raw = (open(rep).read() if rep.endswith(".csv") else  # a saved `--page raw --csv` export
           subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout)
    rows = list(csv.reader(io.StringIO(raw)))
    hdr, data = rows[0], rows[2:]
    c = hdr.index
    layout = " on open-addressing hash tables (HX_JOIN_HASH: the bench's ht_path)" if launches is None else ""
    out = [f"# {tag} — ncu --set full of K1 (k1_probe_agg){layout}, SSB SF{sf}, 1 B200", "",
           "Captured with `ncu --set full --clock-control none --import-source on -k regex:k1_probe_agg "
           f"-s 13 -c 13 python tools/prof_query.py --sf {sf} --queries all --reps 2` (the second, "
           "planned execution of each query). ncu times are cold-cache and serialised: compare shares.", "",
           "| query | kernel | ncu us | algorithmic GB | DRAM r+w GB | traffic/alg | DRAM GB/s (% of 8 TB/s) | L2 hit % | issue active % | warps active % | regs |",
           "|---|---|---|---|---|---|---|---|---|---|---|"]
    def scaled(d, name):  # ncu raw values carry their unit in the second header row
        unit = rows[1][c(name)]
        mult = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9,
                "nsecond": 1e-3, "usecond": 1, "msecond": 1e3, "ns": 1e-3, "us": 1, "ms": 1e3}
        return float(d[c(name)] or 0) * mult.get(unit, 1)

    tt = ta = tr = 0.0
    for q, d in zip(QS, data):
        t = scaled(d, "gpu__time_duration.sum")  # -> us
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
    # speed of light per unit: which resource bounds each launch (ncu % of peak; a launch with no
    # unit near 100% is latency-bound: too few loads in flight for its request pattern)
    sol = [("issue", "smsp__issue_active.avg.pct_of_peak_sustained_active"),
           ("SM", "sm__throughput.avg.pct_of_peak_sustained_elapsed"),
           ("L1TEX", "l1tex__throughput.avg.pct_of_peak_sustained_active"),
           ("L2", "lts__throughput.avg.pct_of_peak_sustained_elapsed"),
           ("DRAM", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed")]
    out += ["", "Speed of light (ncu, % of each unit's peak) and the instruction mix per lineorder row:", "",
            "| query | " + " | ".join(n + " %" for n, _ in sol) + " | top unit | warp instr / row | global-load sectors / row | shared wavefronts / row |",
            "|---|" + "---|" * (len(sol) + 4)]
    for q, d in zip(QS, data):
        v = [float(d[c(m)] or 0) for _, m in sol]
        top = max(range(len(sol)), key=lambda i: v[i])
        inst = float(d[c("smsp__inst_executed.sum")] or 0)
        gld = float(d[c("l1tex__t_sectors_pipe_lsu_mem_global_op_ld.sum")] or 0)
        shw = float(d[c("l1tex__data_pipe_lsu_wavefronts_mem_shared.sum")] or 0)
        out.append(f"| {q} | " + " | ".join(f"{x:.1f}" for x in v) +
                   f" | {sol[top][0]} | {inst / N:.2f} | {gld / N:.3f} | {shw / N:.3f} |")
    with open(os.path.join(ROOT, "profiles", f"{tag}_k1_ncu_summary.md"), "w") as f:
        f.write("\n".join(out) + "\n")
    if launches is None:  # (a capture of another layout: no traffic file, no launch list)
        print("\n".join(out[-20:]))
        return
    with open(os.path.join(ROOT, "profiles", "k1_traffic.json"), "w") as f:
        json.dump({"dram_bytes_per_launch": tr / 13, "algorithmic_bytes_per_launch": ta / 13,
                   "launches": 13, "source": f"profiles/{tag}_k1_ncu_summary.md (ncu --set full, "
                   f"dram__bytes_read.sum + dram__bytes_write.sum, mean over the 13 SSB K1 launches at SF{sf})"}, f, indent=1)
    if probe_csv:
        probe_table(tag, probe_csv, sf)
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


def probe_table(tag, path, sf):
    """Probe-structure L2 hit rate per query from an evict_last-tagged capture."""
    rows = list(csv.reader(open(path)))
    h = [i for i, r in enumerate(rows) if "Kernel Name" in r and "Metric Name" in r][0]
    hd = rows[h]
    per = collections.OrderedDict()
    for r in rows[h + 1:]:
        key = (r[hd.index("ID")], r[hd.index("Kernel Name")].split("(")[0])
        unit = r[hd.index("Metric Unit")] if "Metric Unit" in hd else ""
        mult = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1, "usecond": 1e3,
                "msecond": 1e6, "sector": 1, "Ksector": 1e3, "Msector": 1e6, "Gsector": 1e9}.get(unit, 1)
        per.setdefault(key, {})[r[hd.index("Metric Name")]] = float(r[hd.index("Metric Value")].replace(",", "")) * mult
    L = [f"# {tag} — L2 hit rate of the probe structures, SSB SF{sf}, 1 B200", "",
         "ncu metrics of the 13 K1 launches (`tools/prof_query.py --sf %s --queries all --reps 2`, "
         "second execution) built with probe loads tagged L2::evict_last and gathered measures "
         "L2::evict_first (`tools/build_variant.sh PH -DHX_PROBE_HINT=1 -DHX_GATHER_HINT=1`; the "
         "lineorder stream is evict_first bulk copies). The evict_last sectors are therefore "
         "exactly the lookups of the direct maps / hash-table buckets read from L2 (structures "
         "staged in shared memory make no L2 request)." % sf, "",
         "| query | ncu us | probe sectors (evict_last) | probe L2 hit % | stream+gather sectors (evict_first) | their hit % | DRAM read GB |",
         "|---|---|---|---|---|---|---|"]
    for q, (key, m) in zip(QS, per.items()):
        eh = m.get("lts__t_sectors_srcunit_tex_evict_last_lookup_hit.sum", 0)
        em = m.get("lts__t_sectors_srcunit_tex_evict_last_lookup_miss.sum", 0)
        fh = m.get("lts__t_sectors_srcunit_tex_evict_first_lookup_hit.sum", 0)
        fm = m.get("lts__t_sectors_srcunit_tex_evict_first_lookup_miss.sum", 0)
        t = m.get("gpu__time_duration.sum", 0)
        rd = m.get("dram__bytes_read.sum", 0)
        L.append(f"| {q} | {t/1e3:.1f} | {eh+em:.3g} | {100*eh/max(eh+em,1):.1f} | {fh+fm:.3g} | "
                 f"{100*fh/max(fh+fm,1):.1f} | {rd/1e9:.3f} |")
    with open(os.path.join(ROOT, "profiles", f"{tag}_probe_l2_sf{sf}.md"), "w") as f:
        f.write("\n".join(L) + "\n")
    print("\n".join(L))


if __name__ == "__main__":
    main(*sys.argv[1:6])
