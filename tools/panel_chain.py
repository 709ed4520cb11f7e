import numpy as np, sys
fn = sys.argv[1]
f = open(fn, 'rb').read(); n = 32 * 32 * 24
tr = np.frombuffer(f[:n * 8], dtype=np.uint64).reshape(32, 32, 24).astype(np.float64)
print('per panel chain: factor(J) | CTA J+1: flag, staged, acc, solved, next acc')
tot = 0
for J in range(0, 7):
    c = J + 1
    a = tr[J, J, 3]
    row = ((tr[J, J, 3] - tr[J, J, 2]) / 1e3 if J > 0 else float('nan'), (tr[c, J, 0] - a) / 1e3, (tr[c, J, 1] - tr[c, J, 0]) / 1e3,
           (tr[c, J, 2] - tr[c, J, 1]) / 1e3, (tr[c, J, 3] - tr[c, J, 2]) / 1e3, (tr[c, c, 2] - tr[c, J, 3]) / 1e3)
    print(J, 'factor %.1f | flag+%.1f staged+%.1f acc+%.1f solved+%.1f nextacc+%.1f' % row)
    print('   solve sub-blocks of CTA J+1 (from staged):', ' '.join('%.1f' % ((tr[c, J, i] - tr[c, J, 1]) / 1e3) for i in range(6, 22, 2)))
print('potrf span (CTA0 accready/first -> CTA7 solved): %.1f us' % ((tr[7, 7, 3] - tr[1, 0, 0]) / 1e3))
print('factor CTA J, panel J: per 16-column sub-block (from accready): solved | cross update done; [22] x = b - acc, [23] solve done')
for J in range(1, 8):
    a = tr[J, J, 2]
    print(J, ' '.join('%.1f|%.1f' % ((tr[J, J, 6 + 2 * sb] - a) / 1e3, (tr[J, J, 7 + 2 * sb] - a) / 1e3) for sb in range(8)),
          ' [22] %.1f [23] %.1f' % ((tr[J, J, 22] - a) / 1e3, (tr[J, J, 23] - a) / 1e3))
