"""Interleaved A/B of library builds (development tool): factorization time (median of reps,
CP priority, uniform family seed 0, nb = 960) and a hash of the factor, per n, per build.
Each (build, n) runs in its own process (CHOL_LIB_OVERRIDE); rounds alternate the builds.
  python tools/libab.py 7680,9600,19200 variants/base.so variants/new.so [--rounds 2 --reps 7]"""
import argparse
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
CHILD = r'''
import hashlib, json, os, sys
sys.path.insert(0, %r)
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c
n, reps = int(sys.argv[1]), int(sys.argv[2])
with c.Plan(n, 960, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
    ts = []
    for r in range(reps + 1):
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        if r:
            ts.append(c.chol_last_times(p.h)[0])
    L = np.empty((n, n))
    c.chol_gather(p.h, L, n)
print(json.dumps({"ms": float(np.median(ts)) * 1e3, "best": min(ts) * 1e3,
                  "hash": hashlib.sha256(L.tobytes()).hexdigest()[:12]}))
''' % ROOT

ap = argparse.ArgumentParser()
ap.add_argument("ns")
ap.add_argument("libs", nargs="+")
ap.add_argument("--rounds", type=int, default=2)
ap.add_argument("--reps", type=int, default=7)
a = ap.parse_args()
res = {}
for rnd in range(a.rounds):
    for n in [int(x) for x in a.ns.split(",")]:
        for spec in a.libs:  # path[:VAR=value+VAR2=value...] (extra environment for that build)
            lib, _, extra = spec.partition(":")
            env = dict(os.environ, CHOL_LIB_OVERRIDE=os.path.abspath(lib))
            env.update(kv.split("=", 1) for kv in extra.split("+") if kv)
            out = subprocess.run([sys.executable, "-c", CHILD, str(n), str(a.reps)], env=env, capture_output=True,
                                 text=True, timeout=600)
            if out.returncode:
                print(json.dumps({"lib": spec, "n": n, "error": out.stderr[-400:]}), flush=True)
                continue
            d = json.loads(out.stdout.strip().splitlines()[-1])
            res.setdefault((spec, n), []).append(d)
            print(json.dumps({"round": rnd, "lib": os.path.basename(spec), "n": n, **d}), flush=True)
for (lib, n), v in sorted(res.items(), key=lambda x: (x[0][1], x[0][0])):
    print(f"{n:6d} {os.path.basename(lib):24s} median {min(x['ms'] for x in v):9.3f} ms  best {min(x['best'] for x in v):9.3f}"
          f"  hash {v[0]['hash']}")
