import sys, os
sys.path.insert(0, "/root/repo")
from paper_journals_pvldb_guolst17_b200 import ppr, workload as W
for name in ("tiny", "lj"):
    st, cfg = W.make_stream(name)
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=cfg["eps"])
    h.set_option(ppr.OPT_GRAPHS, 0)
    for _ in range(3):
        s = h.apply_batch(*st.next_batch())
        print(name, "ms_store", s["ms_store"], flush=True)
