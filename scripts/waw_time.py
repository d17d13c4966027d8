#!/usr/bin/env python
"""config3_waw whole jp_schedule call (median, CUDA events) at several densities /
distances: path 9 (default) and, with --restart, the restart form beside it."""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import bench  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
for delta in (1024, 1 << 20):
    for d in (0.001, 0.01, 0.05, 0.10):
        wl = synth.config3_waw(d, delta=delta, device="cuda")
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        res, ms = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st), wl.A, A0, st, 20)
        row = {"d": d, "delta": delta, "ms": round(ms, 4), "G_per_s": round(wl.n / ms / 1e6, 2),
               "path": res["tls_path"], "windows": res["tls"]["windows"]}
        if "--restart" in sys.argv:
            r2, ms2 = bench.median_timed(lambda: jp.jp_schedule(L, ws, stream=st, tls_recovery=1), wl.A, A0, st, 3)
            row.update(restart_ms=round(ms2, 3), restart_windows=r2["tls"]["windows"])
        print(json.dumps(row), flush=True)
        del wl, A0, L, ws
