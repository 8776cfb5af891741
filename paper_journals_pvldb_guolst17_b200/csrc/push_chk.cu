// push_chk.cu -- the Opt push (push.cu) with the exactly-once enqueue check of
// PPR_OPT_CHECK_ENQUEUE (the fused self-update must enqueue each
// (source, vertex) at most once while it is queued).  Every enqueue sets the
// entry's bit in PushArgs::bitmap (unused by Opt) and counts a duplicate if it
// was set; every dequeue clears it before the entry's exchange.  A separate
// build so the production kernels carry none of it.  Exported as
// launch_push_chk; ppr_api.cu picks it when the option is on.
#define PPR_CHECK_ENQ 1
#define PPR_PUSH_OPT_ONLY 1
#define PPR_PUSH_ENTRY launch_push_chk
#include "push.cu"
