"""Whole jp_schedule on config 3 (on-chip grid TLS) for one libjp build
(JP_LIB selects it): median of 7 warm calls per density, CUDA events."""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

out = {"lib": os.path.basename(jp._abi.LIB_PATH)}
for d in (0.001, 0.01, 0.1):
    wl = synth.config3(d, device="cuda")
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    ts, res = [], None
    for _ in range(8):
        wl.A.copy_(A0)
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        res = jp.jp_schedule(L, ws)
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    out[d] = (round(statistics.median(ts[1:]), 4), res["tls"]["windows"], res["tls_w_max"])
    del wl, A0, L, ws
print(out, flush=True)
