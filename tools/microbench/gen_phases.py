"""Regenerate solve_block_T / potf2_block_T in block_phases.cu from tile_ops.cuh, with a
clock64 stamp after every compute barrier (phase timers for the in-block routines)."""
import os
import re

H = os.path.dirname(os.path.abspath(__file__))
src = open(os.path.join(H, '../../paper_conf_ipps_agullobehkmt15_b200/csrc/tile_ops.cuh')).read()
p = os.path.join(H, 'block_phases.cu')
m = open(p).read()


def extract(text, name):
    s = text.index(f'template <int BS>\n__device__ __forceinline__ void {name}(')
    e = text.index('\n}\n', s) + 3
    return s, e


for fn in ['solve_block', 'potf2_block']:
    s, e = extract(src, fn)
    f = src[s:e].replace(f'void {fn}(', f'void {fn}_T(')
    cnt = [0]

    def rep(mm):
        i = cnt[0]
        cnt[0] += 1
        return mm.group(0) + f'\n    if (threadIdx.x == 0) {{ long long _t = clock64(); g_ph[{i}] += _t - g_last; g_last = _t; }}'
    f = re.sub(r'bar_sync\(kBarCompute, kComputeThreads\);[^\n]*', rep, f)
    s2, e2 = extract(m, fn + '_T')
    m = m[:s2] + f + m[e2:]
open(p, 'w').write(m)
