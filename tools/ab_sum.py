"""Summarise an ab_libs.sh output: per build, the sum of per-query K1 medians and each query."""
import re
import sys
for blk in open(sys.argv[1]).read().split('== ')[1:]:
    name, vals = blk.split('\n', 1)
    pairs = re.findall(r'(q\d\.\d) ([\d.]+)', vals)
    tot = sum(float(v) for _, v in pairs)
    print(f"{name.split('/')[-1]:18s} sum {tot:7.3f} ", ' '.join(f"{q[1:]}:{float(v):.3f}" for q, v in pairs))
