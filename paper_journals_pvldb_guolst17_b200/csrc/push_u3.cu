// push_u3.cu -- the Opt push (push.cu) with 3 independent edge chains per lane
// instead of 2, for dense graphs (>= 8 arcs per vertex, the ones the hybrid
// schedule pushes on the ring from the seeds): in-lists there are long enough
// to keep a third load -> load -> atomic chain busy (Orkut-shaped push
// 22.1 -> 21.2 ms), while on sparse graphs (LJ-shaped) it costs registers and
// is 1% slower.  Exported as launch_push_u3; ppr_api.cu picks it.
#define PPR_PUSH_U 3
#define PPR_PUSH_OPT_ONLY 1
#define PPR_PUSH_ENTRY launch_push_u3
#include "push.cu"
