#!/usr/bin/env python
"""DOALL kernel comparison on config 2 (N = 2^28 SAXPY fp32): LDG/STG.128
grid-stride stream vs bulk-copy (TMA) staged ring.  CUDA events, 20 launches
each after 5 warm-ups; prints achieved GB/s (12 B/iteration)."""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

dev = torch.device("cuda:0")
wl = synth.config2(device=dev)
L = jp.Loop.from_workload(wl)
st = torch.cuda.current_stream()
for which in (0, 1, 0, 1):
    jp.jp_doall_kernel(which)
    for _ in range(5):
        jp.jp_schedule(L, None, stream=st)
    ts = []
    for _ in range(20):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        jp.jp_schedule(L, None, stream=st)
        b.record(st)
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    ms = statistics.median(ts)
    print(json.dumps({"kernel": ["ldg128", "tma_bulk"][which], "ms_median": ms, "ms_min": min(ts),
                      "gbs": 12 * wl.n / (ms * 1e-3) / 1e9}), flush=True)
