"""Device time of building one operand form of a b x b tile (vs_form_make), CUDA events around
`iters` back-to-back builds on one stream: python tools/form_time.py [b] [iters]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402  (test infrastructure: an SPD tile's Cholesky factor as input)
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402
import vsgen  # noqa: E402

b = int(sys.argv[1]) if len(sys.argv) > 1 else 1024
iters = int(sys.argv[2]) if len(sys.argv) > 2 else 20
L, _ = oracle.cholesky(vsgen.spd(5, b).astype("float64"))
src = torch.from_numpy(L.astype("float32")).cuda()
for name, f in (("split_rows", 1), ("split_cols", 2), ("inv_l", 3)):
    dst = torch.empty(vs.vs_form_bytes(f, b), dtype=torch.uint8, device="cuda")
    st = torch.cuda.current_stream().cuda_stream
    for _ in range(3):
        vs.vs_form_make(f, b, src.data_ptr(), dst.data_ptr(), st)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(iters):
        vs.vs_form_make(f, b, src.data_ptr(), dst.data_ptr(), st)
    e1.record()
    torch.cuda.synchronize()
    print("%-10s b=%d: %.1f us" % (name, b, e0.elapsed_time(e1) * 1e3 / iters))
