#!/usr/bin/env python
"""Config 1 (N = 4096) as bench.py times it: the wall time of back-to-back
jp_schedule calls (each returns once its results are published), median of 200."""
import os
import statistics
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
for d in (0.0, 0.05):
    wl = synth.config1(d, device="cuda")
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    for _ in range(20):
        jp.jp_schedule(L, ws, stream=st)
    ts = []
    for _ in range(200):
        t0 = time.perf_counter()
        jp.jp_schedule(L, ws, stream=st)
        ts.append(time.perf_counter() - t0)
    torch.cuda.synchronize()
    print({"d": d, "us_per_call": round(statistics.median(ts) * 1e6, 2)}, flush=True)
