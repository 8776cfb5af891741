import os, sys
sys.path.insert(0, os.getcwd())
from paper_journals_pvldb_guolst17_b200 import ppr, workload as W
st, cfg = W.make_stream("tiny")
g0s, g0d = st.window()
s = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
h = ppr.Ppr(cfg["n"], g0s, g0d, s, alpha=0.15, eps=1e-7)
for t in range(3):
    rc, stats = h.apply_batch(*st.next_batch(), raise_on_error=False)
    print("batch", t, rc, ppr.load().ppr_last_error(h._h).decode(), stats["kernel_launches"])
