"""jp_profile_stamp time on config 3 (N = 2^24) for the JP_STAMP_PASS_MB in the env."""
import json, os, sys, statistics
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402
st = torch.cuda.current_stream()
wl = synth.config3(0.01, device="cuda")
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
ref = jp.jp_profile_density(L, ws)
ts = []
for _ in range(8):
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record(st)
    jp.jp_profile_stamp(L, ws, stream=st)
    b.record(st)
    torch.cuda.synchronize()
    ts.append(a.elapsed_time(b))
p = jp.jp_profile_density(L, ws)
assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (ref["raw_iters"], ref["war_iters"], ref["waw_iters"])
print(json.dumps({"pass_mb": os.environ.get("JP_STAMP_PASS_MB", "48"), "stamp_ms": statistics.median(ts),
                  "raw": p["raw_iters"]}))
