#!/usr/bin/env python
"""jp_profile_density wall/event time on config 4 (N = 2^26) and config 3 (d = 1%)."""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

dev = torch.device("cuda:0")
st = torch.cuda.current_stream()
for name, wl in (("config4", synth.config4(device=dev)), ("config3_1pct", synth.config3(0.01, device=dev))):
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    for _ in range(3):
        jp.jp_profile_density(L, ws, stream=st)
    ts = []
    for _ in range(10):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(st)
        jp.jp_profile_density(L, ws, stream=st)
        b.record(st)
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    print(json.dumps({"workload": name, "n": wl.n, "profile_ms_median": statistics.median(ts)}), flush=True)
    del wl, L, ws
