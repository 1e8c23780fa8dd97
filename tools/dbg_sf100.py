import sys, torch, numpy as np
sys.path.insert(0, '/root/repo')
import ssbgen
for sf in (10, 100):
    sz = ssbgen.sizes(sf)
    for c in ssbgen.TABLE_COLS["customer"] + ssbgen.TABLE_COLS["part"]:
        n = ssbgen.table_rows(sz, c)
        t = torch.empty(n, dtype=torch.int32, device="cuda")
        ssbgen.column_device(42, sz, c, t.data_ptr(), 0, n, torch.cuda.current_stream().cuda_stream)
        torch.cuda.synchronize()
        d = t.cpu().numpy(); h = ssbgen.column(42, sz, c)
        bad = np.nonzero(d != h)[0]
        print(sf, c, n, 'mismatches', len(bad), bad[:5], d[bad[:3]] if len(bad) else '', h[bad[:3]] if len(bad) else '')
