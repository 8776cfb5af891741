import numpy as np, sys
sys.path.insert(0, "/root/repo")
import oracle
from paper_journals_pvldb_guolst17_b200 import ppr, workload as W
st, cfg = W.make_stream("tiny")
g0s, g0d = st.window()
srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 2)
b = st.next_batch()
res = {}
for S in (1, 2):
    for sf in (0, 1):
        for mode in ("opt",):
            h = ppr.Ppr(cfg["n"], g0s, g0d, srcs[:S], alpha=0.15, eps=1e-7)
            h.set_option(ppr.OPT_PUSH, 0)
            h.set_option(ppr.OPT_SMALL_FRONT, sf)
            o = oracle.Oracle(cfg["n"], g0s, g0d, srcs[:S], 0.15, 1e-7)
            for i in range(S):
                P, R = h.query(i); o.set_state(i, P, R)
            h.apply_batch(*b); o.apply(*b, do_push=False)
            for i in range(S):
                P, R = h.query(i); Po, Ro = o.query(i)
                d = np.abs(R - Ro); k = np.argmax(d)
                print(f"S={S} small_front={sf} src{i}: max|dR|={d.max():.3e} at v={k} R={R[k]:.6e} Ro={Ro[k]:.6e} dout gpu/orc={h.export_dout()[k]}/{o.dout()[k]} eqP={np.array_equal(P,Po)}")
            print("  dout equal:", np.array_equal(h.export_dout(), o.dout()), "arcs equal:", all(np.array_equal(x,y) for x,y in zip(h.export_edges(), o.export())))
