#!/usr/bin/env python
"""Privatized stream comparison on config 4 (N = 2^26 PRIV_TMP fp32, S = 1024):
LDG/STG.128 kernel vs bulk-copy (TMA) staged kernel (jp_doall_kernel selects
both).  jp_run_privatized timed with CUDA events; 12 B/iteration."""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

dev = torch.device("cuda:0")
wl = synth.config4(device=dev)
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
st = torch.cuda.current_stream()
prof = jp.jp_profile_density(L, ws)
for which in (0, 1, 0, 1):
    jp.jp_doall_kernel(which)
    for _ in range(5):
        jp.jp_run_privatized(L, prof, ws, stream=st)
    ts = []
    for _ in range(20):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        jp.jp_run_privatized(L, prof, ws, stream=st)
        b.record(st)
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    ms = statistics.median(ts)
    print(json.dumps({"kernel": ["ldg128", "tma_bulk"][which], "ms_median": ms, "ms_min": min(ts),
                      "gbs": 12 * wl.n / (ms * 1e-3) / 1e9}), flush=True)
