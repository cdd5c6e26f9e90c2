import json, sys
for f in sys.argv[1:]:
    for l in open(f):
        if l.startswith('{'):
            d = json.loads(l); r = d.get('roofline', {})
            print(f, d['config'].get('workload'), 'ms', round(d['ms_per_step'], 4), 'frac', round(r.get('frac', 0), 3),
                  d.get('result_digest'))
