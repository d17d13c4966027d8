"""Whole jp_schedule() on config 3 with the interleaved classify tables on / off
(JP_CLASSIFY_PAIRS), CUDA events, median of 7 warm calls.  Usage: python scripts/classify_pairs.py"""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

for d in (0.001, 0.01, 0.1):
    wl = synth.config3(d, device="cuda")
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    row = {}
    for pairs in ("0", "1", "0", "1"):
        os.environ["JP_CLASSIFY_PAIRS"] = pairs
        ts = []
        for _ in range(8):
            wl.A.copy_(A0)
            torch.cuda.synchronize()
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record()
            jp.jp_schedule(L, ws)
            b.record()
            torch.cuda.synchronize()
            ts.append(a.elapsed_time(b))
        row["pairs" + pairs] = round(statistics.median(ts[1:]), 4)
    print({"density": d, **row}, flush=True)
    del wl, A0, L, ws
