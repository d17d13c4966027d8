import os
import sys

R = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path[:0] = [R, os.path.join(R, "tests")]
import torch  # noqa: E402

import oracle as O  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402
from helpers import to_oracle  # noqa: E402

dev = torch.device("cuda:0")
n = int(sys.argv[1])
d = float(sys.argv[2])
W = int(sys.argv[3]) if len(sys.argv) > 3 else 4096
wl = synth.config3(d, n=n)
st, A, _, stats = O.sim_tls(to_oracle(wl), W)
g = wl.to(dev)
r0, w0 = g.r.clone(), g.w.clone()
L = jp.Loop.from_workload(g)
got = jp.jp_run_tls(L, window=W, w_max=4096, path=1, ws=jp.workspace(L))
torch.cuda.synchronize()
print("nbad", int((g.A.cpu().numpy() != A).sum()), "stats_eq", got == stats, got["windows"], stats["windows"],
      "indices intact", torch.equal(r0, g.r), torch.equal(w0, g.w), flush=True)
