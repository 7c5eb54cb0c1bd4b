"""Per-warp timeline of the history kernel's two phases (dev variant NT_TIMELINE=1).

NT_LIB_VARIANT=tl python scripts/dev/phase_timeline.py [config] [out.json]
Each warp stamps (globaltimer ns) its start, the moment its refill finds the particle range
exhausted, and its end.  Reported per phase: the launch span, when the range ran out
(first warp to see it), and the quantiles of warp end times -- i.e. how much of each phase
is the tail in which warps only finish the histories they hold.
"""
import ctypes as C
import json
import os
import sys
from pathlib import Path

import numpy as np

ROOT = Path(__file__).resolve().parents[2]
sys.path.insert(0, str(ROOT))
from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl  # noqa: E402

cfgname = sys.argv[1] if len(sys.argv) > 1 else "csp"
out = sys.argv[2] if len(sys.argv) > 2 else None
cfg = wl.CONFIGS[cfgname]
L = binding.lib()
f = L.nt_dev_timeline
f.argtypes = [C.c_void_p]
res = {"config": cfgname}
for step in range(3):                       # warm-up steps, the last one is reported
    t = binding.setup(cfg, device=0, mode="history")
    s = t.run_timestep(cfg.dt)
    buf = np.zeros((2, 8192, 3), dtype=np.uint64)
    assert f(buf.ctypes.data) == 0
    t.close()
for ph in range(2):
    b = buf[ph].astype(np.int64)
    live = b[:, 0] > 0
    b = b[live]
    t0 = b[:, 0].min()
    st, ex, en = (b[:, 0] - t0) / 1e3, (b[:, 1] - t0) / 1e3, (b[:, 2] - t0) / 1e3   # us
    ex = np.where(b[:, 1] > 0, ex, np.nan)
    span = en.max()
    first_ex = np.nanmin(ex)
    q = {p: float(np.percentile(en, p)) for p in (10, 25, 50, 75, 90, 99, 100)}
    res[f"phase{ph + 1}"] = {
        "warps": int(live.sum()), "span_us": float(span), "range_exhausted_at_us": float(first_ex),
        "tail_us": float(span - first_ex), "tail_frac": float((span - first_ex) / span),
        "warp_end_quantiles_us": q,
        "warp_busy_frac": float(np.mean(en - st) / span),
    }
res["track_ms"] = s["track_ms"]
print(json.dumps(res, indent=1))
if out:
    Path(out).write_text(json.dumps(res, indent=1))
