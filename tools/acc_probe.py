"""Accuracy of the fp32-class tile versions against the oracle as the tile grows (relF on sampled
rows for MATMUL; full tiles for TRSM / POTRF).  python tools/acc_probe.py"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.environ.get("GRAFT_REPO_ROOT", os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import oracle  # noqa: E402
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402
import vsgen  # noqa: E402


def run(t, v, b, arrays):
    ts = [torch.from_numpy(np.ascontiguousarray(x)).cuda() for x in arrays]
    info = torch.zeros(1, dtype=torch.int32, device="cuda")
    vs.vs_tile_run(t, v, b, [x.data_ptr() for x in ts], info.data_ptr())
    torch.cuda.synchronize()
    return [x.cpu().numpy() for x in ts]


for b in (1024, 2048, 4096):
    A, B, C0 = (vsgen.uniform(800 + i, b, b) for i in range(3))
    rows = [0, 255, 256, b // 2 - 1, b - 1]
    ref = oracle.matmul(A[rows], B, C0[rows])
    for v in (vs.VS_V_TC_3XF16, vs.VS_V_TC_3XTF32, vs.VS_V_SIMT_F32):
        C = run(vs.VS_T_MATMUL, v, b, [A, B, C0])[2]
        print(b, "MATMUL", vs.VERSION_NAMES[v], "relF %.2e" % oracle.relF(C[rows], ref), flush=True)
for b in (1024, 2048):
    S = vsgen.spd(900 + b, b, np.float64)
    Lref, _ = oracle.cholesky(S)
    X0 = vsgen.uniform(901, b, b)
    xref = oracle.trsm(Lref.astype(np.float32), X0)
    for v in (vs.VS_V_TC_3XTF32, vs.VS_V_TC_3XF16):
        X = run(vs.VS_T_TRSM, v, b, [Lref.astype(np.float32), X0])[1]
        print(b, "TRSM", vs.VERSION_NAMES[v], "relF %.2e" % oracle.relF(X, xref), flush=True)
    L = run(vs.VS_T_POTRF, vs.VS_V_TC_3XTF32, b, [S.astype(np.float32)])[0]
    lo = np.tril_indices(b)
    print(b, "POTRF tc_3xtf32 relF %.2e" % oracle.relF(L[lo], Lref[lo]), flush=True)
