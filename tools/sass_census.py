"""SASS op census of libhx.so (cuobjdump -sass): per kernel family, the instructions that show
the design — bulk copies (UBLKCP), mbarrier ops (SYNCS), shared-memory loads (LDS), global
loads (LDG), L2 prefetch (UBLKPF / CCTL), tensor-core ops (HMMA/UTCMMA: none expected).

    python tools/sass_census.py [libhx.so] > profiles/r02_sass_census.md
"""
import collections
import re
import subprocess
import sys

lib = sys.argv[1] if len(sys.argv) > 1 else "paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so"
out = subprocess.run(["cuobjdump", "-sass", lib], capture_output=True, text=True).stdout
fam, counts = None, collections.defaultdict(collections.Counter)
OPS = ["UBLKCP", "UBLKPF", "SYNCS", "LDS", "STS", "LDG", "STG", "ATOMS", "ATOMG", "RED", "SHFL",
       "VOTE", "BAR", "HMMA", "UTCMMA", "UTCHMMA", "UTCQMMA"]
for line in out.splitlines():
    m = re.search(r"Function : (\S+)", line)
    if m:
        name = m.group(1)
        for k in ("k1_probe_agg", "k1_scan_agg", "k1_prepare", "k1_finalize", "k2_", "k3_", "ssbgen"):
            if k in name:
                fam = k.rstrip("_")
                break
        else:
            fam = "other"
        counts[fam]["kernels"] += 1
        continue
    m = re.search(r"/\*[0-9a-f]+\*/\s+(?:@!?U?P\w+\s+)?([A-Z][A-Z0-9_]*)(\.[A-Z0-9_.]*)?", line)
    if m and fam:
        op = m.group(1)
        for o in OPS:
            if op == o or op.startswith(o + "_"):
                counts[fam][o] += 1
print("# SASS op census of libhx.so (sm_100a), `python tools/sass_census.py`\n")
print("Static instruction counts per kernel family (all template instances summed). UBLKCP = "
      "cp.async.bulk (TMA bulk engine), SYNCS = mbarrier operations; no HMMA/UTC*MMA: nothing "
      "on the path is a dense contraction.\n")
print("| family | kernels | " + " | ".join(OPS) + " |")
print("|---|---|" + "---|" * len(OPS))
for f, c in sorted(counts.items()):
    print(f"| {f} | {c['kernels']} | " + " | ".join(str(c[o]) for o in OPS) + " |")
