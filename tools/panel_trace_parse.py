import sys, struct
import numpy as np
f = open(sys.argv[1], 'rb').read()
n = 32 * 32 * 24
tr = np.frombuffer(f[:n * 8], dtype=np.uint64).reshape(32, 32, 24).astype(np.float64)
ck = np.frombuffer(f[n * 8:2 * n * 8], dtype=np.int64).reshape(32, 32, 24)
vals = [tr[c, J, i] for c in range(8) for J in range(c + 1) for i in range(6) if tr[c, J, i] > 0]
t0 = min(vals)
print("cta panel | eflag Lstaged accready solved | pflag plast   (us from first event)")
for c in range(8):
    for J in range(c + 1):
        print("%3d %5d |" % (c, J) + "".join(" %8.1f" % ((tr[c, J, i] - t0) / 1e3 if tr[c, J, i] > 0 else -1) for i in range(6)))
print("factor (CTA J, panel J): us, MHz")
for c in range(8):
    us = (tr[c, c, 3] - tr[c, c, 2]) / 1e3
    cy = ck[c, c, 3] - ck[c, c, 2]
    print(c, "%.1f us" % us, "%.0f MHz" % (cy / us if us > 0 else 0))
print("end:", (max(vals) - t0) / 1e3)
print("sb0 of the factor: tmem->x, solve done (before stores), solved (after stores)   us from accready")
for c in range(1, 8):
    a = tr[c, c, 2]
    print(c, "%.1f %.1f %.1f" % ((tr[c, c, 22] - a) / 1e3, (tr[c, c, 23] - a) / 1e3, (tr[c, c, 6] - a) / 1e3))
