"""One line per bench JSON: workload, value, roofline frac, per-width (variant, us)."""
import json
import sys

for path in sys.argv[1:]:
    try:
        d = json.loads(open(path).read().strip().splitlines()[-1])
    except Exception as e:  # noqa: BLE001
        print(path, "unreadable:", e)
        continue
    pw = d.get("per_width") or {}
    print(path.split("/")[-1], "%.0f %s" % (d["value"], d["unit"]), "frac=%.3f" % d["roofline"]["frac"],
          "e2e=%s" % (round(d["e2e"]["value"]) if d.get("e2e") else None),
          {k: (v["variant"], round(v["us"], 2)) for k, v in pw.items()} if pw else d["config"].get("variant", ""))
