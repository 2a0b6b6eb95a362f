"""Print SASS (with executed counts and stall samples) around given line indices of
one launch of an .ncu-rep:  ncu_sass_ctx.py REP SKIP IDX[,IDX...] [RADIUS]"""
import csv, subprocess, sys
path, skip, idxs = sys.argv[1], int(sys.argv[2]), [int(x) for x in sys.argv[3].split(',')]
rad = int(sys.argv[4]) if len(sys.argv) > 4 else 12
out = subprocess.run(['ncu', '-i', path, '--page', 'source', '--csv', '--print-source', 'sass',
                      '--launch-skip', str(skip), '--launch-count', '1'], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
hdr = rows[1]
ie = hdr.index('Instructions Executed'); src = hdr.index('Source'); ss = hdr.index('Warp Stall Sampling (All Samples)')
seen = set(); uniq = []
for r in rows[2:]:
    if len(r) != len(hdr) or r[0] in seen: continue
    seen.add(r[0]); uniq.append(r)
for i in idxs:
    print(f'---- around {i}')
    for j in range(max(0, i - rad), min(len(uniq), i + 4)):
        r = uniq[j]
        print(f'{j:5d} {r[src][:70]:70s} inst={r[ie]:>9s} samp={r[ss]}')
