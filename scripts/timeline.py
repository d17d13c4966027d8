#!/usr/bin/env python
"""GPU timeline of one whole jp_schedule call (CUPTI through torch.profiler):
every kernel / memset / memcpy with its start offset, duration and the idle gap
before it -- where a call's time goes besides its kernels.

  python scripts/timeline.py [config3|config4|config5] [d]
"""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402
from torch.profiler import ProfilerActivity, profile  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

cfg = sys.argv[1] if len(sys.argv) > 1 else "config3"
d = float(sys.argv[2]) if len(sys.argv) > 2 else 0.01
st = torch.cuda.current_stream()
if cfg == "config3":
    wl = synth.config3(d, device="cuda")
    kw = {}
elif cfg == "config4":
    wl = synth.config4(device="cuda")
    kw = {}
else:
    wl = synth.config5(device="cuda")
    kw = {"scheme": jp.JP_SCHED_STEALING, "chunk_iters": 65536}
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for _ in range(3):
    wl.A.copy_(A0)
    jp.jp_schedule(L, ws, stream=st, **kw)
torch.cuda.synchronize()
wl.A.copy_(A0)
torch.cuda.synchronize()
with profile(activities=[ProfilerActivity.CUDA, ProfilerActivity.CPU]) as prof:
    a = torch.cuda.Event(enable_timing=True)
    b = torch.cuda.Event(enable_timing=True)
    a.record(st)
    jp.jp_schedule(L, ws, stream=st, **kw)
    b.record(st)
    torch.cuda.synchronize()
ms = a.elapsed_time(b)
path = os.path.join(ROOT, "gpurun_out", f"timeline_{cfg}.json")
os.makedirs(os.path.dirname(path), exist_ok=True)
prof.export_chrome_trace(path)
ev = json.load(open(path))["traceEvents"]
gpu = [e for e in ev if e.get("ph") == "X" and e.get("cat") in ("kernel", "gpu_memset", "gpu_memcpy")]
gpu.sort(key=lambda e: e["ts"])
t0 = gpu[0]["ts"] if gpu else 0
end = t0
print(f"{cfg} d={d}: call {ms * 1e3:.1f} us between events; {len(gpu)} GPU activities")
busy = 0.0
for e in gpu:
    gap = e["ts"] - end
    print(f"  +{e['ts'] - t0:8.1f}  {e['dur']:7.1f} us  gap {gap:6.1f}  s{e['args'].get('stream', '?'):>3}  {e['name'][:80]}")
    end = max(end, e["ts"] + e["dur"])
    busy += e["dur"]
print(f"  span {end - t0:.1f} us, sum of durations {busy:.1f} us")
